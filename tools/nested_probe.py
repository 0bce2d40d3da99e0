"""Speed of nested ||| fan-out vs running each nested ||| inside one thread."""
import os
import sys
import torch
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from paper_conf_cluster_subdbn18_b200 import culi, workloads as W  # noqa: E402

culi.load()
defs = "\n".join([W.FIB_DEF, "(define pfib (lambda (xs) (||| (length xs) fib xs)))",
                  "(define xs '(%s))" % " ".join(["15"] * 4096)])
forms = "\n".join(["(length (pfib xs))"] * 16)            # 16 forms x 4096 elements x fib(15)
for flags, name in ((0, "nested fan-out"), (culi.CULI_F_NO_NESTED, "sequential in-thread")):
    ctx = culi.Context(stream=torch.cuda.current_stream().cuda_stream, flags=flags)
    ctx.define(defs)
    h = ctx.upload(forms)
    ctx.eval_uploaded(h)
    ts = []
    for _ in range(3):
        ctx.eval_uploaded(h)
        ms, _, _ = ctx.last_timing()
        ts.append(ms[1])
    r = ctx.fetch_results(h)
    total, nerr = r.totals()
    print("%-22s %9.2f ms  %7.2f G steps/s  results %s  nested=%s" %
          (name, min(ts), total / min(ts) / 1e6, r.printed()[:2], ctx.last_stats() and ctx.last_nested))
    ctx.close()
