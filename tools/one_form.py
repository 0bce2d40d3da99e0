"""Evaluate one form (argv[1], text) a few times after the fib definition — for ncu captures."""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from paper_conf_cluster_subdbn18_b200 import culi
from paper_conf_cluster_subdbn18_b200 import workloads as W
culi.load()
ctx = culi.Context(device=0, stream=torch.cuda.current_stream().cuda_stream)
ctx.define(W.FIB_DEF)
form = sys.argv[1]
if form.startswith("@"):
    kind, n = form[1:].split(":")
    form = {"carlist": "(car (list %s))", "c0": "(||| %s fib (%%s))" % n}[kind] % " ".join(["5"] * int(n))
for _ in range(int(sys.argv[2]) if len(sys.argv) > 2 else 3):
    r = ctx.eval_batch(form)
    ms, k, _ = ctx.last_timing()
    print(r.printed()[0][:40], ms)
