#!/bin/bash
# Session-2 check at HEAD: build, GPU suite once, bench lines C0-C5.  Under gpurun.
cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()" > $OUT/s2a_build.log 2>&1 || { echo build failed; exit 1; }
timeout 1200 python -m pytest tests -m gpu -x -q -p no:cacheprovider --timeout 600 > $OUT/s2a_pytest.log 2>&1; echo "suite rc=$? $(tail -1 $OUT/s2a_pytest.log)"
python -c "import __graft_entry__ as g; g.smoke()" > $OUT/s2a_smoke.log 2>&1; echo "smoke rc=$? $(tail -1 $OUT/s2a_smoke.log)"
for WL in ${WLS:-C0 C1 C2 C3 C4 C5}; do timeout 900 python bench.py --workload $WL --steps 10 --warmup 3 > $OUT/s2a_bench_$WL.json 2> $OUT/s2a_bench_$WL.err; python -c "import json;d=json.load(open('$OUT/s2a_bench_$WL.json'));print('$WL', round(d['value']), {k: round(v,3) for k,v in d['phases_ms'].items()}, 'e2e', round(d['e2e']['value']), 'clk', d['clocks'])"; done
