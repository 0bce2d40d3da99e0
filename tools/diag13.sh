cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
for v in 1024 4096 16384; do
  for WL in C2 C5; do CULI_SPLIT_SLEEP=$v timeout 600 python bench.py --workload $WL --steps 5 --warmup 3 --e2e-steps 1 --no-cpu-baseline 2>/dev/null | python -c "import json,sys;d=json.loads(sys.stdin.read());print('sleep $v $WL', d['phases_ms'], d['value'])"; done
done
