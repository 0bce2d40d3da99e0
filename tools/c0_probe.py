"""C0 anatomy: eval-phase time of (||| n fib L) with L an evaluated data list vs a quoted list, for several n,
and variants that isolate the pieces of a wide list below the top level.  Run on the GPU box."""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from paper_conf_cluster_subdbn18_b200 import culi
from paper_conf_cluster_subdbn18_b200 import workloads as W
culi.load()
ctx = culi.Context(device=0, stream=torch.cuda.current_stream().cuda_stream)
ctx.define(W.FIB_DEF)
def t(form, reps=5):
    best = 1e9
    for _ in range(reps):
        r = ctx.eval_batch(form)
        ms, k, _ = ctx.last_timing()
        best = min(best, ms[1])
    ctx.last_stats()
    return round(best, 4), ctx.last_nested
for n in [int(a) for a in (sys.argv[1:] or ["256", "1024", "4096"])]:
    L = " ".join(["5"] * n)
    print(n, "data", t("(||| %d fib (%s))" % (n, L)), "quoted", t("(||| %d fib '(%s))" % (n, L)),
          "bare", t("(%s)" % L), "len-list", t("(length (list %s))" % L), "car-list", t("(car (list %s))" % L),
          "len-quoted", t("(length '(%s))" % L), "car-data", t("(car (1 %s))" % L),
          "plus", t("(+ %s)" % L))
