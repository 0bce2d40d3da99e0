#!/bin/bash
# Round-end measurement refresh: bench lines for C1-C5 (+ C0 / reference), launch list and ncu full capture
# of the C2 eval kernel, eval_inst_c2.json for bench.py's roofline.  Under gpurun.
OUT=gpurun_out; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1 || exit 1
for WL in ${WLS:-C1 C2 C3 C4 C5}; do
  timeout 900 python bench.py --workload $WL > $OUT/final_$WL.json 2> $OUT/final_$WL.err
  python -c "import json;d=json.load(open('$OUT/final_$WL.json'));print('$WL', round(d['value']), 'forms/s', round(d['eval_steps_per_sec']/1e9,2), 'Gsteps/s', {k: round(v,3) for k,v in d['phases_ms'].items()}, 'e2e', round(d['e2e']['value']), 'cpu', d['cpu_baseline'] and round(d['cpu_baseline']['value']), 'reader_ms', round(d['reader']['ms'],3))"
done
if [ -z "$SKIP_NCU" ]; then
  timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file $OUT/launches_C2.csv python bench.py --workload C2 --steps 2 --warmup 1 --e2e-steps 1 --no-cpu-baseline > /dev/null 2>&1
  python tools/ncu_summary.py launches $OUT/launches_C2.csv > $OUT/launches_C2.md
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:culi_eval_kernel -s 1 -c 1 -o $OUT/prof_C2 -f python bench.py --workload C2 --steps 1 --warmup 1 --e2e-steps 1 --no-cpu-baseline > /dev/null 2>&1
  python tools/ncu_summary.py full $OUT/prof_C2.ncu-rep --json $OUT/eval_inst_c2.json > $OUT/prof_C2_summary.txt 2>&1
  head -3 $OUT/launches_C2.md
fi
