"""C4 anatomy: eval-phase time vs batch size (throughput- or tail-bound?), voting on/off.
Usage: python tools/c4_probe.py N [novote]"""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from paper_conf_cluster_subdbn18_b200 import culi
from paper_conf_cluster_subdbn18_b200 import workloads as W
culi.load()
n = int(sys.argv[1])
flags = culi.CULI_F_NO_VOTING if "novote" in sys.argv else 0
ctx = culi.Context(device=0, stream=torch.cuda.current_stream().cuda_stream, flags=flags)
wl = W.c4(n)
ctx.define(wl.defs)
h = ctx.upload(wl.forms)
best = 1e9
for _ in range(5):
    ctx.eval_uploaded(h)
    torch.cuda.synchronize()
    ms, k, _ = ctx.last_timing()
    best = min(best, ms[1])
res = ctx.fetch_results(h)
tot = sum(res.steps())
print("novote" if flags else "voting", n, "eval %.3f ms" % best, "%.1f M forms/s" % (n / best / 1e3),
      "%.2f G steps/s" % (tot / best / 1e6), flush=True)
