"""Separate per-warp latency from throughput: time batches of identical (fib k) forms of growing size."""
import os
import sys
import torch
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from paper_conf_cluster_subdbn18_b200 import culi, workloads as W  # noqa: E402

culi.load()
ctx = culi.Context(stream=torch.cuda.current_stream().cuda_stream, heap_nodes=1 << 24)
ctx.define(W.FIB_DEF)
for k, n in [(22, 32), (22, 256), (22, 1024), (22, 8192), (22, 32768), (22, 65536), (18, 65536)]:
    h = ctx.upload("\n".join(["(fib %d)" % k] * n))
    for _ in range(2):
        ctx.eval_uploaded(h)
    ts = []
    for _ in range(3):
        ctx.eval_uploaded(h)
        ms, _, _ = ctx.last_timing()
        ts.append(ms[1])
    steps = 27 * [0, 1, 1, 2, 3, 5, 8, 13, 21, 34, 55, 89, 144, 233, 377, 610, 987, 1597, 2584, 4181, 6765, 10946,
                  17711, 28657][k + 1] - 17
    t = min(ts)
    print("fib(%d) x %6d: %8.2f ms  %7.2f Gsteps/s  %6.0f cycles/step/warp@1.965GHz" %
          (k, n, t, steps * n / t / 1e6, t * 1e-3 * 1.965e9 / steps))
    ctx.release(h)
