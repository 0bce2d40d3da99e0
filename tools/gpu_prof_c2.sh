cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT
timeout 900 ncu --set full --import-source on --clock-control none -k regex:culi_eval_kernel -c 1 -o $OUT/r2_prof_C2 python bench.py --workload C2 --steps 1 --warmup 1 --e2e-steps 1 --no-cpu-baseline > $OUT/r2_prof_C2.log 2>&1
ls -la $OUT/r2_prof_C2*
python tools/ncu_summary.py full $OUT/r2_prof_C2.ncu-rep > $OUT/r2_prof_C2_summary.txt 2>&1; cat $OUT/r2_prof_C2_summary.txt | head -60
ncu -i $OUT/r2_prof_C2.ncu-rep --page source --csv --print-source sass > $OUT/r2_prof_C2_sass.csv 2>/dev/null; ls -la $OUT/r2_prof_C2_sass.csv
