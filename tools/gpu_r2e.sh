cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT
for WL in C5 C4 C2; do timeout 600 python bench.py --workload $WL --steps 5 --warmup 3 --e2e-steps 1 --no-cpu-baseline > $OUT/r2e_bench_$WL.json 2> $OUT/r2e_bench_$WL.err; python -c "import json;d=json.load(open('$OUT/r2e_bench_$WL.json'));print('$WL', d['value'], d['phases_ms'], d['e2e']['value'])"; done
