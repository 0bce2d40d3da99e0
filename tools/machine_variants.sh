#!/bin/bash
# Bench C2/C5 with alternative eval machines: tools/variants/<name>.patch applied to culi_machine.cuh
# (round-1 experiments kept as diffs; "head" = the file as it is).  Under gpurun.
M=paper_conf_cluster_subdbn18_b200/csrc/culi_machine.cuh
cp $M /tmp/machine_orig.cuh
for v in ${MV:-head spec}; do
  cp /tmp/machine_orig.cuh $M
  if [ "$v" != head ]; then patch -s $M < tools/variants/$v.patch || { echo "patch failed $v"; continue; }; fi
  python -c "import sys; sys.path.insert(0,'paper_conf_cluster_subdbn18_b200'); import build; build.build(force=True)" > /dev/null 2>&1 || { echo "build failed $v"; continue; }
  for w in ${WLS:-C2 C5}; do
    python bench.py --workload $w --steps 5 --warmup 3 --e2e-steps 1 --no-cpu-baseline 2>/dev/null | tail -1 | python -c "import json,sys;d=json.loads(sys.stdin.readline());print('$v $w eval %.2f ms' % d['phases_ms']['eval'])"
  done
done
cp /tmp/machine_orig.cuh $M
