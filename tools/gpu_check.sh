#!/bin/bash
# Build, GPU suite once, smoke, bench lines for $WLS (default C0 C2 C4 C5).  TAG names the outputs.  Under gpurun.
cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
OUT=gpurun_out; mkdir -p $OUT; TAG=${TAG:-chk}
python -c "import __graft_entry__ as g; g.build()" > $OUT/${TAG}_build.log 2>&1 || { echo build failed; tail $OUT/${TAG}_build.log; exit 1; }
if [ -z "$NO_SUITE" ]; then
timeout 1200 python -m pytest tests -m gpu -x -q -p no:cacheprovider --timeout 600 > $OUT/${TAG}_pytest.log 2>&1; echo "suite rc=$? $(tail -1 $OUT/${TAG}_pytest.log)"
grep -E "FAILED|Error" $OUT/${TAG}_pytest.log | head -5
python -c "import __graft_entry__ as g; g.smoke()" > $OUT/${TAG}_smoke.log 2>&1; echo "smoke rc=$? $(tail -1 $OUT/${TAG}_smoke.log)"
fi
for WL in ${WLS:-C0 C2 C4 C5}; do timeout 900 python bench.py --workload $WL --steps 10 --warmup 3 $BENCH_ARGS > $OUT/${TAG}_bench_$WL.json 2> $OUT/${TAG}_bench_$WL.err; python -c "import json;d=json.load(open('$OUT/${TAG}_bench_$WL.json'));print('$WL', round(d['value']), {k: round(v,3) for k,v in d['phases_ms'].items()}, 'e2e', round(d['e2e']['value']), 'clk', d['clocks']['sm_mhz'], d['clocks']['reasons'])" || tail -3 $OUT/${TAG}_bench_$WL.err; done
