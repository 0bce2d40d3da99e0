#!/bin/bash
# Small-batch experiment: eval-phase time of C1 / C4 / C3 with argument splitting on (0) and off (32),
# and with a shorter idle-warp back-off cap.  Run on a GPU box from the repo root.
mkdir -p gpurun_out
for w in C1 C4 C3 C0; do
  for f in 0 32; do
    python bench.py --workload $w --steps 10 --warmup 3 --no-cpu-baseline --flags $f --e2e-steps 1 2>/dev/null \
      | python -c "import json,sys; d=json.loads(sys.stdin.readline()); print('$w', 'flags=$f', round(d['ms_per_step'],4), d['phases_ms'])"
  done
  CULI_SPLIT_SLEEP=512 python bench.py --workload $w --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 1 2>/dev/null \
      | python -c "import json,sys; d=json.loads(sys.stdin.readline()); print('$w', 'sleep=512', round(d['ms_per_step'],4), d['phases_ms'])"
done
