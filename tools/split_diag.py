"""Split diagnostics: eval-phase time, splits and bounded-wait give-ups of one workload, for A/B builds
(CULI_LIB=path/to/libculi.so).  python tools/split_diag.py C2 [flags] [reps]"""
import os, sys, time, faulthandler
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
faulthandler.dump_traceback_later(int(os.environ.get("DIAG_TIMEOUT", "100")), exit=True)
import torch
from paper_conf_cluster_subdbn18_b200 import culi, workloads as W
L = culi.load()
if os.environ.get("DIAG_PIDFILE"):
    open(os.environ["DIAG_PIDFILE"], "w").write(str(os.getpid()))
wlname = sys.argv[1]
flags = int(sys.argv[2]) if len(sys.argv) > 2 else 0
reps = int(sys.argv[3]) if len(sys.argv) > 3 else 5
n = int(os.environ.get("DIAG_N", "0"))
wl = {"C2": lambda: W.c2(n or 65536), "C5": lambda: W.c5(n or 20000), "C4": lambda: W.c4(n or 262144),
      "C1": lambda: W.c1(n or 1024)}[wlname]()
s = torch.cuda.Stream()
kw = {} if wlname == "C2" else dict(heap_nodes=1 << 28)
ctx = culi.Context(stream=s.cuda_stream, flags=flags, **kw)
if wl.defs:
    ctx.define(wl.defs)
h = ctx.upload(wl.forms)
evs = []
t0 = time.time()
for k in range(reps):
    ctx.eval_uploaded(h)
    ms, kern, _ = ctx.last_timing()
    evs.append(ms[1]); disp = ms[0]
r = ctx.fetch_results(h)
tot, nerr = r.totals()
sp = ctx.last_splits()
w = ctx.last_waits() if hasattr(L, "culi_last_waits") else None
cl = ctx.last_split_claims() if hasattr(L, "culi_last_split_claims") else None
print("%s flags=%d lib=%s dispatch %.3f eval ms %s steps %d err %d splits %d claimed %s waits %s wall %.1fs" % (
    wlname, flags, os.path.basename(os.environ.get("CULI_LIB", "libculi.so")), disp, " ".join("%.2f" % e for e in evs),
    tot, nerr, sp, cl, w, time.time() - t0), flush=True)
