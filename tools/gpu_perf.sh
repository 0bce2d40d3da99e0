#!/bin/bash
# One GPU iteration: build, GPU tests, bench (WLS), ncu full capture of the eval kernel on C2 with the
# stall and hot-footprint summaries.  Under gpurun.  SKIP_TESTS=1 / SKIP_NCU=1 to skip parts.
OUT=gpurun_out; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1 || { tail -20 $OUT/build.log; exit 1; }
if [ -z "$SKIP_TESTS" ]; then
  timeout 900 python -m pytest tests -m gpu -x -q > $OUT/pytest_gpu.log 2>&1; echo "pytest rc=$?" >> $OUT/pytest_gpu.log
  tail -2 $OUT/pytest_gpu.log
fi
for WL in ${WLS:-C2 C5}; do
  timeout 900 python bench.py --workload $WL --steps ${STEPS:-5} --no-cpu-baseline --e2e-steps 1 > $OUT/bench_$WL.json 2> $OUT/bench_$WL.err; tail -2 $OUT/bench_$WL.err
  python -c "import json;d=json.load(open('$OUT/bench_$WL.json'));print('$WL', round(d['value']), 'forms/s', round(d['eval_steps_per_sec']/1e9,2), 'Gsteps/s eval', round(d['phases_ms']['eval'],3), 'ms')"
done
if [ -z "$SKIP_NCU" ]; then
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:culi_eval_kernel -s 1 -c 1 -o $OUT/prof_C2 -f python bench.py --workload C2 --steps 1 --warmup 1 --e2e-steps 1 --no-cpu-baseline > $OUT/ncu_full.log 2>&1
  python tools/ncu_summary.py full $OUT/prof_C2.ncu-rep --json $OUT/eval_inst_c2.json > $OUT/prof_C2_summary.txt 2>&1
  ncu -i $OUT/prof_C2.ncu-rep --page source --csv --print-source sass > $OUT/sass.csv 2>/dev/null
  ncu -i $OUT/prof_C2.ncu-rep --page source --csv --print-source cuda,sass > $OUT/src.csv 2>/dev/null
  python tools/hot_footprint.py $OUT/sass.csv | tee $OUT/footprint.txt
  python tools/stalls.py $OUT/src.csv > $OUT/stalls.txt 2>&1; head -12 $OUT/stalls.txt
  grep -E "inst_executed.sum|issue_active|time_duration" $OUT/prof_C2_summary.txt
fi
