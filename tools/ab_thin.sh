cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
for r in 1 2; do for V in 32 8 4 2 0; do for WL in C1; do
  CULI_THIN_LANES=$V timeout 600 python bench.py --workload $WL --steps 20 --warmup 3 --e2e-steps 1 --no-cpu-baseline 2>/dev/null | python -c "import json,sys;d=json.loads(sys.stdin.read());print('lanes=$V $WL eval %.4f step %.4f value %.4g' % (d['phases_ms']['eval'], d['ms_per_step'], d['value']))"
done; done; done
