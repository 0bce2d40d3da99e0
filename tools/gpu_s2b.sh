#!/bin/bash
# C0 (paper-shaped) eval: launch list + ncu full of the eval kernel with source.  Under gpurun.
cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/s2b_build.log 2>&1 || { echo build failed; exit 1; }
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 300 --csv --log-file $OUT/s2b_launches_C0.csv python bench.py --workload C0 --steps 2 --warmup 1 --e2e-steps 1 --no-cpu-baseline > /dev/null 2>&1
python tools/ncu_summary.py launches $OUT/s2b_launches_C0.csv > $OUT/s2b_launches_C0.md; head -20 $OUT/s2b_launches_C0.md
TAG=s2b WLS=C0 bash tools/gpu_prof.sh
python tools/stalls.py $OUT/s2b_prof_C0_sass.csv | head -40
