cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
for r in 1 2; do for V in 1 0; do for WL in C4 C1; do
  CULI_SIZE_FIRST=$V timeout 600 python bench.py --workload $WL --steps 5 --warmup 3 --e2e-steps 1 --no-cpu-baseline 2>/dev/null | python -c "import json,sys;d=json.loads(sys.stdin.read());print('size_first=$V $WL eval %.3f dispatch %.3f value %.4g' % (d['phases_ms']['eval'], d['phases_ms']['dispatch'], d['value']))"
done; done; done
