cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -p no:cacheprovider -k "quasiquote or paper_examples or edge or random_programs or defun" 2>&1 | tail -3
for L in "" scratch/libculi_leafcall.so; do
  for WL in C2 C5 C4; do CULI_LIB=$L timeout 600 python bench.py --workload $WL --steps 5 --warmup 3 --e2e-steps 1 --no-cpu-baseline 2>/dev/null | python -c "import json,sys;d=json.loads(sys.stdin.read());print('lib=${L:-default} $WL', d['phases_ms']['eval'], d['value'])"; done
done
