import sys, os
sys.path.insert(0, os.getcwd())
import torch
from paper_conf_cluster_subdbn18_b200 import culi
from paper_conf_cluster_subdbn18_b200 import workloads as W
culi.load()
defs = "\n".join([W.FIB_DEF, W.FACT_DEF, W.WHEN_DEF, W.C3_DEFS_HEAD[0], W.C3_DEFS_HEAD[1]])
forms = "\n".join(["(* 2 (+ 4 3) 6)", "(+ 1 2)", "(||| 3 + (1 2 3) (4 5 6))", "(fib 5)", "(fact 20)", "(when (< 1 2) 5)",
    "(||| 4 f '(0.5 -1.25 3.0 2.5))", "(list (fib 10) (fact 10) (reverse (list 1 2 3)))"] + ["(fib %d)" % (n % 12) for n in range(256)])
ctx = culi.Context(device=0, stream=torch.cuda.current_stream().cuda_stream, slots=148 * 128, heap_nodes=1 << 22, vstack_entries=1024)
ctx.define(defs)
for i in range(4):
    r = ctx.eval_batch(forms)
    print(i, ctx.last_timing()[0])
