#!/bin/bash
# tests + bench for several workloads (no ncu).  Usage: WLS="C2 C3" bash tools/gpu_quick.sh
OUT=gpurun_out; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1
if [ -z "$SKIP_TESTS" ]; then
  timeout 900 python -m pytest tests -m gpu -x -q > $OUT/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> $OUT/pytest_gpu.log
  tail -4 $OUT/pytest_gpu.log
fi
for WL in ${WLS:-C2}; do
  timeout 900 python bench.py --workload $WL $BENCH_ARGS > $OUT/bench_$WL.json 2> $OUT/bench_$WL.err; tail -2 $OUT/bench_$WL.err
  python -c "import json;d=json.load(open('$OUT/bench_$WL.json'));print('$WL', round(d['value']), 'forms/s', round(d['eval_steps_per_sec']/1e9,2), 'Gsteps/s', d['phases_ms'], 'e2e', round(d['e2e']['value']))"
done
