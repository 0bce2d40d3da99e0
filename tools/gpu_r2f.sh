cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT
for i in 1 2 3 4 5; do timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider --timeout 600 > $OUT/r2f_pytest_$i.log 2>&1; echo "run $i rc=$? $(tail -1 $OUT/r2f_pytest_$i.log)"; done | tee $OUT/r2f_suite5.txt
timeout 1500 bash tools/hang_probe.sh 20 > $OUT/r2f_hang20.txt 2>&1; echo "hang probe lines: $(grep -c ' ok ' $OUT/r2f_hang20.txt) ok, $(grep -c FAIL $OUT/r2f_hang20.txt) fail, waits: $(grep -o 'waits_gave_up [0-9]*' $OUT/r2f_hang20.txt | sort | uniq -c)"
for WL in C0 C1 C2 C3 C4 C5; do timeout 900 python bench.py --workload $WL --steps 10 --warmup 3 > $OUT/r2f_bench_$WL.json 2> $OUT/r2f_bench_$WL.err; python -c "import json;d=json.load(open('$OUT/r2f_bench_$WL.json'));print('$WL', round(d['value']), d['phases_ms'], 'e2e', round(d['e2e']['value']), 'cpu', d['cpu_baseline'] and round(d['cpu_baseline']['value']))"; done
