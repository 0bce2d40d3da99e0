# ncu --set full of the eval kernel for workloads $WLS (default C2 C5); summary + SASS source page.
cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT; TAG=${TAG:-r2}
for WL in ${WLS:-C2 C5}; do
  timeout 900 ncu --set full --import-source on --clock-control none -k regex:"culi_eval" -c 1 -o $OUT/${TAG}_prof_$WL python bench.py --workload $WL --steps 1 --warmup 1 --e2e-steps 1 --no-cpu-baseline $BENCH_ARGS > $OUT/${TAG}_prof_$WL.log 2>&1
  python tools/ncu_summary.py full $OUT/${TAG}_prof_$WL.ncu-rep > $OUT/${TAG}_prof_${WL}_summary.txt 2>&1; head -25 $OUT/${TAG}_prof_${WL}_summary.txt
  ncu -i $OUT/${TAG}_prof_$WL.ncu-rep --page source --csv --print-source sass > $OUT/${TAG}_prof_${WL}_sass.csv 2>/dev/null
  ncu -i $OUT/${TAG}_prof_$WL.ncu-rep --page raw --csv > $OUT/${TAG}_prof_${WL}_raw.csv 2>/dev/null
done
