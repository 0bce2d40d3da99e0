"""Small batches over every language feature, run under compute-sanitizer (tools/sanitize.sh)."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from paper_conf_cluster_subdbn18_b200 import culi, workloads as W  # noqa: E402

culi.load()
defs = "\n".join([W.FIB_DEF, W.FACT_DEF, W.SUM_DEF, W.SUM_LIST_DEF] + W.C4_MACROS + W.C3_DEFS_HEAD +
                 ["(define xs '(0.5 1.5 -2.0 3.25))"])
edge = [l.split("\t")[0] for l in open(os.path.join(ROOT, "tests/golden/edge_cases.tsv"))
        if l.strip() and not l.startswith("#")]
forms = "\n".join(edge + W.c1(64).form_lines() + W.c2(64, lo=3, hi=9).form_lines() +
                  W.c4(256).form_lines() + W.c5(512).form_lines() + ["(||| 4 f xs)", "(||| 3 + '(1 2 3) '(4 5 6))"])
ctx = culi.Context(slots=148 * 128, heap_nodes=1 << 22, vstack_entries=1024)
ctx.define(defs)
for flags in (0, culi.CULI_F_NO_BINNING | culi.CULI_F_NO_FANOUT):
    c2 = culi.Context(slots=148 * 128, heap_nodes=1 << 22, vstack_entries=1024, flags=flags)
    c2.define(defs)
    r = c2.eval_batch(forms)
    print(len(r), r.totals())
    c2.close()
# device reader (§8(f)2) incl. strings, quotes, comments, floats needing the big-integer path, and heap
# reclamation (§8(f)3) after the definitions
text = forms + "\n" + "\n".join(['"a (b) ; c"', "'(x . y)", "; comment\n(list 1 2.5 \"s\")",
                                   "1.00000000000000000000000000000000000001e-300", "(quote (1 (2 (3))))"])
for flags in (0, culi.CULI_F_NO_GC):
    c3 = culi.Context(slots=148 * 128, heap_nodes=1 << 22, vstack_entries=1024, flags=flags)
    c3.define_text(defs)
    c3.define_text("(define tmp (list 1 2 3))\n(define tmp (reverse tmp))")
    c3.collect()
    r = c3.eval_text(text)
    print(len(r), r.totals(), c3.heap_usage())
    c3.close()
# setq (mutable mode, R7) and CUDA-graph replay on a non-default stream
import torch  # noqa: E402
st = torch.cuda.Stream()
c4 = culi.Context(slots=148 * 128, heap_nodes=1 << 22, vstack_entries=1024, stream=st.cuda_stream)
c4.define("(define make-counter (lambda () (let ((n 0)) (lambda () (setq n (+ n 1))))))\n(define g 1)\n(setq g 2)")
r = c4.eval_batch("(let ((c (make-counter))) (c) (c))\n(let ((acc 0)) (||| 3 (lambda (x) (setq acc (+ acc x))) '(1 2 3)) acc)\n(setq g 5)")
print(r.printed())
h = c4.upload(forms)
for _ in range(3):
    c4.eval_uploaded(h)
print(c4.fetch_results(h).totals())
c4.release(h)
c4.close()
# nested ||| and wide lists below the top level (NEST_EVAL), incl. an element error
c5 = culi.Context(slots=148 * 128, heap_nodes=1 << 22, vstack_entries=1024)
c5.define(W.FIB_DEF + "\n(define pfib (lambda (xs) (||| (length xs) fib xs)))\n" +
          "(define wl (lambda (k) (list %s)))" % " ".join("(* k %d)" % i for i in range(70)))
wide = " ".join(["5"] * 300)
r = c5.eval_batch("\n".join(["(||| 300 fib (%s))" % wide, "(length (wl 3))", "(pfib '(%s))" % wide,
                              "(car (list %s))" % " ".join(["(fib 6)"] * 100),
                              "(1 %s)" % " ".join(["(car 5)"] * 80)]))
print(r.printed()[1], r.totals(), c5.last_stats())
c5.close()
print("done")
