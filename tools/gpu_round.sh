#!/bin/bash
# One GPU session: tests, bench, ncu launch list + full capture of the eval kernel.  Run under gpurun.
set -x
OUT=gpurun_out
mkdir -p $OUT
WL=${WL:-C2}
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1
if [ -z "$SKIP_TESTS" ]; then
  timeout 900 python -m pytest tests -m gpu -x -q > $OUT/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> $OUT/pytest_gpu.log
  tail -5 $OUT/pytest_gpu.log
fi
timeout 600 python bench.py --workload $WL > $OUT/bench_$WL.json 2> $OUT/bench_$WL.err; tail -3 $OUT/bench_$WL.err; cat $OUT/bench_$WL.json
if [ -z "$SKIP_NCU" ]; then
  timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file $OUT/launches_$WL.csv python bench.py --workload $WL --steps 2 --warmup 1 --e2e-steps 1 --no-cpu-baseline > $OUT/ncu_launch_bench.log 2>&1
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:${KREGEX:-culi_eval_kernel} -s 1 -c 1 -o $OUT/prof_$WL -f python bench.py --workload $WL --steps 1 --warmup 1 --e2e-steps 1 --no-cpu-baseline > $OUT/ncu_full.log 2>&1
  tail -3 $OUT/ncu_full.log
fi
if [ -f $OUT/prof_$WL.ncu-rep ]; then
  python tools/ncu_summary.py full $OUT/prof_$WL.ncu-rep --json $OUT/eval_inst_$(echo $WL | tr A-Z a-z).json > $OUT/prof_${WL}_summary.txt 2>&1
  python tools/ncu_summary.py launches $OUT/launches_$WL.csv > $OUT/launches_${WL}.md 2>&1
  cat $OUT/eval_inst_$(echo $WL | tr A-Z a-z).json
fi
