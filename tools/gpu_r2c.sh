cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT
timeout 400 python bench.py --steps 10 --warmup 3 > $OUT/r2c_bench_c2.json 2> $OUT/r2c_bench_c2.err; tail -3 $OUT/r2c_bench_c2.err
for WL in C1 C3 C4 C5; do timeout 600 python bench.py --workload $WL --steps 10 --warmup 3 > $OUT/r2c_bench_$WL.json 2> $OUT/r2c_bench_$WL.err; tail -2 $OUT/r2c_bench_$WL.err; done
timeout 300 python bench.py --workload C4 --steps 10 --warmup 3 --flags 8 --no-cpu-baseline > $OUT/r2c_bench_C4_novote.json 2> $OUT/r2c_bench_C4_novote.err
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,smsp__thread_inst_executed_per_inst_executed.ratio,lts__t_sector_hit_rate.pct,smsp__issue_active.avg.pct_of_peak_sustained_active,smsp__inst_executed.sum,sm__warps_active.avg.pct_of_peak_sustained_active,l1tex__t_bytes_pipe_lsu_mem_local_op_ld.sum,l1tex__t_bytes_pipe_lsu_mem_local_op_st.sum
for WL in C1 C2 C3 C4 C5; do
  timeout 900 ncu --metrics $M --clock-control none --csv -k regex:"culi_eval|culi_fanout_kernel" -c 3 --log-file $OUT/r2c_sweep_$WL.csv python bench.py --workload $WL --steps 1 --warmup 1 --e2e-steps 1 --no-cpu-baseline > $OUT/r2c_sweep_$WL.log 2>&1
done
timeout 300 ncu --metrics $M --clock-control none --csv -k regex:"culi_eval" -c 3 --log-file $OUT/r2c_sweep_C4novote.csv python bench.py --workload C4 --flags 8 --steps 1 --warmup 1 --e2e-steps 1 --no-cpu-baseline > $OUT/r2c_sweep_C4novote.log 2>&1
timeout 300 ncu --metrics gpu__time_duration.sum --clock-control none --csv -c 400 --log-file $OUT/r2c_launches_c2.csv python bench.py --steps 2 --warmup 1 --e2e-steps 1 --no-cpu-baseline > $OUT/r2c_launches_c2.log 2>&1
python tools/ncu_summary.py sweep $OUT/r2c_sweep_*.csv > $OUT/r2c_sweep.md 2>&1; cat $OUT/r2c_sweep.md
