"""GPU tests of heap reclamation ("marked as free"): after every culi_define
the persistent segment is compacted to what the global environment reaches.  Results (values, steps,
errors) must equal the oracle's and those of a session without reclamation (CULI_F_NO_GC); the segment
must shrink to the reachable nodes and stay bounded under repeated redefinition; contiguous spines must
stay contiguous (the ||| fan-out still takes its O(1) path)."""
from __future__ import annotations

import os

import pytest

from paper_conf_cluster_subdbn18_b200 import workloads as W
from tests.parity import compare

pytestmark = pytest.mark.gpu

SMALL = dict(slots=148 * 128, heap_nodes=1 << 24, vstack_entries=2048)

DEFS = "\n".join([
    W.FIB_DEF, W.FACT_DEF, W.SUM_DEF, W.SUM_LIST_DEF, W.WHEN_DEF,
    "(define junk (length (append (list 1 2 3 4 5 6 7 8) (reverse (list 9 10 11 12)))))",
    "(define make-adder (lambda (k) (lambda (x) (+ x k))))",
    "(define add5 (make-adder 5))",
    "(define g (let ((a 1.5) (b 2) (c 'sym) (d (list 1 2)) (e \"str ing\")) (lambda (x) (list a b c d e x))))",
    "(define dl (cons 1 (cons 2 (cons 3 nil))))",
    "(define dp (cons 1 2.5))",
    "(define sh (let ((x (list 1 2))) (list x x)))",
    "(define s \"hello world\")",
    "(define xs (list 1 2 3 4 5 6 7 8 9 10 11 12 13 14 15 16 17 18 19 20 21 22 23 24 25 26 27 28 29 30 31 32 33 34 35 36 37 38 39 40))",
    "(define ys '(0.5 1.5 2.5 3.5 4.5 5.5 6.5 7.5 8.5 9.5 10.5 11.5 12.5 13.5 14.5 15.5 16.5 17.5 18.5 19.5 20.5 21.5 22.5 23.5 24.5 25.5 26.5 27.5 28.5 29.5 30.5 31.5 32.5 33.5))",
    "(define nested (list (list 1 (list 2 3)) (cons 'a 'b) (list \"s\" 4.25)))",
    "(defmacro swap-args (f a b) (list f b a))",
])
FORMS = "\n".join([
    "(fib 15)", "(fact 20)", "(sum 100)", "(sum-list xs)", "(when (< 1 2) 5)", "junk", "(add5 10)",
    "(g 7)", "dl", "dp", "(eq (car sh) (car (cdr sh)))", "sh", "s", "(length xs)", "(||| 40 add5 xs)",
    "(||| 34 (lambda (y) (* y 2.0)) ys)", "nested", "(swap-args - 1 10)", "(make-adder 3)",
    "((make-adder 3) 4)", "(car (cdr (car nested)))", "(equal nested (list (list 1 (list 2 3)) (cons 'a 'b) (list \"s\" 4.25)))",
])


@pytest.fixture(scope="module")
def culi():
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_cluster_subdbn18_b200 import culi as C
    from paper_conf_cluster_subdbn18_b200 import build
    build.build()
    C.load()
    return C


def test_results_unchanged_and_segment_shrinks(culi, oracle_mod):
    on = culi.Context(**SMALL)
    off = culi.Context(**SMALL, flags=culi.CULI_F_NO_GC)
    on.define(DEFS)
    off.define(DEFS)
    used_on, _, freed = on.heap_usage()
    used_off, _, freed_off = off.heap_usage()
    assert freed > 0 and freed_off == 0
    assert used_on + freed == used_off                  # every node is either kept or reclaimed
    assert used_on < used_off
    a, b = on.eval_batch(FORMS), off.eval_batch(FORMS)
    assert a.printed() == b.printed() and a.steps() == b.steps()
    s = oracle_mod.Session()
    s.define(DEFS)
    bad = compare(a.printed(), a.steps(), s.eval(FORMS), FORMS.splitlines())
    assert not bad, "\n".join(bad)
    # compacted spines are still contiguous: both ||| forms fan out, none falls back
    on.eval_batch("(||| 40 add5 xs)\n(||| 34 (lambda (y) (* y 2.0)) ys)")
    assert on.last_stats() == (2, 0)


def test_collect_is_idempotent(culi):
    ctx = culi.Context(**SMALL)
    ctx.define(DEFS)
    used, _, _ = ctx.heap_usage()
    live, freed = ctx.collect()
    assert freed == 0 and live + 2 == used
    assert ctx.heap_usage()[0] == used


def test_redefinition_stays_bounded(culi, oracle_mod):
    ctx = culi.Context(**SMALL)
    body = " ".join(str(i) for i in range(500))
    sizes = []
    for k in range(30):
        ctx.define("(define big (list %s %d))\n(define tmp (reverse big))\n(define f%d (lambda (x) (+ x %d)))"
                   % (body, k, k % 3, k))
        sizes.append(ctx.heap_usage()[0])
    assert max(sizes[5:]) == min(sizes[5:])               # steady state: old versions are reclaimed
    res = ctx.eval_batch("(length big)\n(car (reverse tmp))\n(f0 1)\n(f1 1)\n(f2 1)")
    assert res.printed() == ["501", "0", "28", "29", "30"]


def test_define_text_and_c3(culi, oracle_mod):
    """configs[2]'s 1M-float list through the device reader, then reclamation: the ||| still fans out."""
    wl = W.c3(1 << 16)
    ctx = culi.Context(**{**SMALL, "heap_nodes": 1 << 24})
    ctx.define_text(wl.defs)
    _, _, freed = ctx.heap_usage()
    assert freed > 0                                    # the define forms themselves are garbage
    res = ctx.eval_batch(wl.forms)
    assert ctx.last_stats() == (1, 0)
    s = oracle_mod.Session()
    s.define(wl.defs)
    bad = compare(res.printed(), res.steps(), s.eval(wl.forms))
    assert not bad, bad


def test_workloads_with_and_without_gc(culi, oracle_mod):
    for wl in (W.c4(3000), W.c5(5000)):
        a = culi.Context(**SMALL)
        b = culi.Context(**SMALL, flags=culi.CULI_F_NO_GC)
        for c in (a, b):
            c.define(wl.defs)
        ra, rb = a.eval_batch(wl.forms), b.eval_batch(wl.forms)
        assert ra.printed() == rb.printed() and ra.steps() == rb.steps()


def test_define_failure_then_collect(culi):
    ctx = culi.Context(**SMALL)
    ctx.define("(define keep (list 1 2 3))")
    with pytest.raises(culi.CuliError):
        ctx.define("(define a (list 4 5))\n(define b (car 5))\n(define c 3)")
    res = ctx.eval_batch("keep\na\nb\nc")
    assert res.printed() == ["(1 2 3)", "(4 5)", "b", "c"]
