"""Timeline of one wide-list suspension (variant build with -DCULI_NEST_TRACE=1): owner suspend, first
claim, last element done, owner resume (globaltimer ns), for (car (list 5 ... 5))."""
import sys, os, ctypes
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from paper_conf_cluster_subdbn18_b200 import build, culi
from paper_conf_cluster_subdbn18_b200 import workloads as W
lib = build.build(defines=["CULI_NEST_TRACE=%s" % os.environ.get("TRACE_LEVEL", "1")] + (["CULI_SLEEP_GATE=1"] if os.environ.get("GATE") else []), out=os.path.join(os.path.dirname(__file__), "..", "gpurun_out", "libculi_trace.so"))
L = culi.load(lib)
ctx = culi.Context(device=0, stream=torch.cuda.current_stream().cuda_stream)
ctx.define(W.FIB_DEF)
T = (ctypes.c_ulonglong * 8)()
for n in (256, 4096, 16384):
    for form in ("(car (list %s))", "(||| %d fib (%%s))" % n):
        f = form % " ".join(["5"] * n)
        for rep in range(3):
            L.culi_debug_nest_trace_reset()
            ctx.eval_batch(f)
            torch.cuda.synchronize()
            L.culi_debug_nest_trace(T)
            ms, _, _ = ctx.last_timing()
            t = list(T)
            print(n, form[:10], "eval %.3f ms" % ms[1], "start->DATA_START %.1f us" % ((t[6] - t[5]) / 1e3),
                  "count %.1f us" % ((t[7] - t[6]) / 1e3), "count->suspend %.1f us" % ((t[3] - t[7]) / 1e3),
                  "suspend->claim %.1f us" % ((t[0] - t[3]) / 1e3),
                  "claim->lastdone %.1f us" % ((t[1] - t[0]) / 1e3), "lastdone->resume %.1f us" % ((t[2] - t[1]) / 1e3),
                  "claims / warm recount end", t[4], "warm recount %.1f us" % ((t[4] - t[7]) / 1e3) if t[4] > 1e12 else "")
