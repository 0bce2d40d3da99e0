"""Argument-splitting probe: eval-kernel time of C2 (and optionally C5 / a fib(22)-only
batch) with splitting off and on at several poll periods / back-off caps.  Run on a GPU box:
    python tools/split_probe.py [C2|C5|FIB22] ..."""
from __future__ import annotations

import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import torch  # noqa: E402

from paper_conf_cluster_subdbn18_b200 import culi  # noqa: E402
from paper_conf_cluster_subdbn18_b200 import workloads as W  # noqa: E402


def run(wl, flags=0, poll=None, sleep=None, reps=3):
    for k, v in (("CULI_SPLIT_POLL", poll), ("CULI_SPLIT_SLEEP", sleep)):
        if v is None:
            os.environ.pop(k, None)
        else:
            os.environ[k] = str(v)
    ctx = culi.Context(device=0, stream=torch.cuda.current_stream().cuda_stream, flags=flags)
    ctx.define(wl.defs)
    best = None
    for _ in range(reps):
        r = ctx.eval_batch(wl.forms)
        ms = ctx.last_timing()[0][1]
        best = ms if best is None else min(best, ms)
    steps = sum(r.steps())
    out = (best, ctx.last_splits(), steps / best / 1e6)
    ctx.close()
    return out


def main():
    which = sys.argv[1:] or ["C2"]
    culi.load()
    for name in which:
        if name == "C2":
            wl = W.c2()
        elif name == "C5":
            wl = W.c5(1 << 20)
        else:
            wl = W.c2(8192, lo=22, hi=23)
        base = run(wl, culi.CULI_F_NO_SPLIT)
        print("%s no-split: eval %.2f ms  %.1f G steps/s" % (name, base[0], base[2]), flush=True)
        for poll in (16, 64, 256):
            for sleep in (4096,):
                ms, sp, gs = run(wl, 0, poll, sleep)
                print("%s split poll=%d sleep=%d: eval %.2f ms  groups %d  %.1f G steps/s  (x%.2f)"
                      % (name, poll, sleep, ms, sp, gs, base[0] / ms), flush=True)


if __name__ == "__main__":
    main()
