#!/bin/bash
# Build libculi.so with several -D flag sets and bench each (C2 by default).  Under gpurun.
# Usage: VARIANTS="base|-DCULI_STAGE_CODE=1" WL=C2 bash tools/variants.sh
OUT=gpurun_out; mkdir -p $OUT
WL=${WL:-C2}
IFS='|' read -ra VS <<< "${VARIANTS:-base}"
for v in "${VS[@]}"; do
  flags=""; [ "$v" != "base" ] && flags="$v"
  CULI_EXTRA_FLAGS="$flags" python -c "
import os, sys; sys.path.insert(0, 'paper_conf_cluster_subdbn18_b200')
import build
build.FLAGS += [f for f in os.environ.get('CULI_EXTRA_FLAGS', '').split() if f]
build.build(force=True)
" > $OUT/build_variant.log 2>&1 || { echo "build failed: $v"; tail -5 $OUT/build_variant.log; continue; }
  timeout 600 python bench.py --workload $WL --steps ${STEPS:-5} --warmup 3 --e2e-steps 1 --no-cpu-baseline > $OUT/v.json 2> $OUT/v.err
  python -c "import json;d=json.load(open('$OUT/v.json'));print('%-40s %s %8.0f forms/s %6.2f Gsteps/s eval %.3f ms' % ('$v', '$WL', d['value'], d['eval_steps_per_sec']/1e9, d['phases_ms']['eval']))" || tail -3 $OUT/v.err
done
