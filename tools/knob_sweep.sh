#!/bin/bash
# Eval-phase time of one workload under environment knobs (CULI_SPLIT_FIRST, CULI_SPLIT_POLL, ...).
# Usage (under gpurun): WL=C2 KNOB=CULI_SPLIT_FIRST VALUES="1 2 4 64" bash tools/knob_sweep.sh
WL=${WL:-C2}
for v in ${VALUES:-64}; do
  env $KNOB=$v python bench.py --workload $WL --steps ${STEPS:-5} --warmup 3 --e2e-steps 1 --no-cpu-baseline $BENCH_ARGS 2>/dev/null | tail -1 | \
    python -c "import json,sys;d=json.loads(sys.stdin.readline());print('$WL $KNOB=$v eval %.3f ms, step %.3f ms, %.1f Gsteps/s, splits %s, waits %s' % (d['phases_ms']['eval'], d['ms_per_step'], d['eval_steps_per_sec']/1e9, d.get('split_groups'), d.get('waits_gave_up')))"
done
