#!/bin/bash
# Session-2 measurement refresh (under gpurun): ncu sweep of the eval-phase kernels C0-C5 ->
# profiles/eval_inst_<cfg>.json (bench.py's traffic / issue numbers), bench lines C0-C5, the C2 launch list,
# a full ncu capture of the C2 eval kernel (+ stall reasons), and the oracle reference arm on C2.
cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT; T=${TAG:-s2}
python -c "import __graft_entry__ as g; g.build()" > $OUT/${T}_build.log 2>&1 || { echo build failed; exit 1; }
if [ -z "$SKIP_SWEEP" ]; then
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,smsp__thread_inst_executed_per_inst_executed.ratio,lts__t_sector_hit_rate.pct,smsp__issue_active.avg.pct_of_peak_sustained_active,smsp__inst_executed.sum,sm__warps_active.avg.pct_of_peak_sustained_active,l1tex__t_bytes_pipe_lsu_mem_local_op_ld.sum,l1tex__t_bytes_pipe_lsu_mem_local_op_st.sum
for WL in ${WLS:-C0 C1 C2 C3 C4 C5}; do
  timeout 1200 ncu --metrics $M --clock-control none --csv -k regex:"culi_eval_kernel|culi_eval_vote|culi_fanout_kernel|culi_export|culi_flat" \
    -c ${COUNT:-12} --log-file $OUT/${T}_sweep_$WL.csv python bench.py --workload $WL --steps 1 --warmup 1 --e2e-steps 1 \
    --no-cpu-baseline > $OUT/${T}_sweep_$WL.log 2>&1
done
python tools/ncu_summary.py sweep $OUT/${T}_sweep_C*.csv > $OUT/${T}_sweep.md 2>&1
python tools/ncu_summary.py profiles profiles $OUT/${T}_sweep_C*.csv
cat $OUT/${T}_sweep.md
fi
for WL in ${BWLS:-C0 C1 C2 C3 C4 C5}; do
  timeout 900 python bench.py --workload $WL --steps 10 --warmup 3 > $OUT/${T}_bench_$WL.json 2> $OUT/${T}_bench_$WL.err
  python -c "import json;d=json.load(open('$OUT/${T}_bench_$WL.json'));print('$WL', round(d['value']), round(d['eval_steps_per_sec']/1e9,2), 'Gsteps/s', {k: round(v,3) for k,v in d['phases_ms'].items()}, 'e2e', round(d['e2e']['value']), 'cpu', d['cpu_baseline'] and round(d['cpu_baseline']['value']), 'clk', d['clocks'])" || tail -3 $OUT/${T}_bench_$WL.err
done
if [ -z "$SKIP_NCU" ]; then
  timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file $OUT/${T}_launches_c2.csv python bench.py --workload C2 --steps 2 --warmup 1 --e2e-steps 1 --no-cpu-baseline > /dev/null 2>&1
  python tools/ncu_summary.py launches $OUT/${T}_launches_c2.csv > $OUT/${T}_launches_c2.md; head -6 $OUT/${T}_launches_c2.md
  timeout 900 ncu --set full --import-source on --clock-control none -k regex:culi_eval_kernel -s 1 -c 1 -o $OUT/${T}_prof_C2 -f python bench.py --workload C2 --steps 1 --warmup 1 --e2e-steps 1 --no-cpu-baseline > /dev/null 2>&1
  python tools/ncu_summary.py full $OUT/${T}_prof_C2.ncu-rep > $OUT/${T}_eval_c2_ncu_full.txt 2>&1
  ncu -i $OUT/${T}_prof_C2.ncu-rep --page source --csv --print-source cuda,sass > $OUT/${T}_prof_C2_src.csv 2>/dev/null
  python tools/stalls.py $OUT/${T}_prof_C2_src.csv > $OUT/${T}_eval_c2_stalls.txt 2>&1; head -12 $OUT/${T}_eval_c2_stalls.txt
fi
timeout 900 python bench.py --impl reference --workload C2 --steps 2 --warmup 1 > $OUT/${T}_bench_C2_reference.json 2>/dev/null; tail -c 300 $OUT/${T}_bench_C2_reference.json
