# A/B eval-phase time of two builds: LIBS="a.so b.so" WLS="C2 C4" REPS=2 bash tools/ab.sh  (under gpurun)
cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
for r in $(seq 1 ${REPS:-2}); do
for L in ${LIBS}; do
  for WL in ${WLS:-C2 C4 C5}; do
    LL=$L; [ "$L" = default ] && LL=""
    CULI_LIB=$LL timeout 600 python bench.py --workload $WL --steps 5 --warmup 3 --e2e-steps 1 --no-cpu-baseline $BENCH_ARGS 2>/dev/null | python -c "import json,sys;d=json.loads(sys.stdin.read());print('$L $WL eval %.3f dispatch %.3f value %.4g' % (d['phases_ms']['eval'], d['phases_ms']['dispatch'], d['value']))"
  done
done
done
