cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT
timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider --timeout 600 > $OUT/r2d_pytest.log 2>&1; echo "pytest rc=$?" >> $OUT/r2d_pytest.log; tail -3 $OUT/r2d_pytest.log
CULI_SHARE_DEVICE=1 CULI_DIST_BACKEND=gloo timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29511 bench.py --gpus 2 --steps 3 --warmup 3 --e2e-steps 1 > $OUT/r2d_bench_n2.json 2> $OUT/r2d_bench_n2.err; echo "n2 rc=$?"; tail -c 1500 $OUT/r2d_bench_n2.json; tail -5 $OUT/r2d_bench_n2.err
for WL in C4 C5; do timeout 600 python bench.py --workload $WL --steps 10 --warmup 3 > $OUT/r2d_bench_$WL.json 2> $OUT/r2d_bench_$WL.err; python -c "import json;d=json.load(open('$OUT/r2d_bench_$WL.json'));print('$WL', d['value'], d['phases_ms'], d['e2e']['value'])"; done
