#!/bin/bash
# ncu metrics of the eval-phase kernels for every config (HBM GB/s, warp execution
# efficiency, L2 hit rate, issue utilisation, local-memory traffic) + the device reader kernels on C5.
# Under gpurun.  Output: gpurun_out/sweep_<WL>.csv and gpurun_out/sweep.md
OUT=gpurun_out; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/build.log 2>&1 || exit 1
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,smsp__thread_inst_executed_per_inst_executed.ratio,lts__t_sector_hit_rate.pct,smsp__issue_active.avg.pct_of_peak_sustained_active,smsp__inst_executed.sum,sm__warps_active.avg.pct_of_peak_sustained_active,l1tex__t_bytes_pipe_lsu_mem_local_op_ld.sum,l1tex__t_bytes_pipe_lsu_mem_local_op_st.sum
for WL in ${WLS:-C1 C2 C3 C4 C5}; do
  timeout 1200 ncu --metrics $M --clock-control none --csv -k regex:"culi_eval_kernel|culi_fanout_kernel|culi_export|culi_flat|rd::" \
    -c ${COUNT:-40} --log-file $OUT/sweep_$WL.csv python bench.py --workload $WL --steps 1 --warmup 1 --e2e-steps 1 \
    --no-cpu-baseline > $OUT/sweep_$WL.log 2>&1
done
python tools/ncu_summary.py sweep $OUT/sweep_*.csv > $OUT/sweep.md 2>&1
cat $OUT/sweep.md
