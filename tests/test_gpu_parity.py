"""GPU parity: the CUDA path (through the C-ABI) against the oracle, element by element, on seeded
synthetic batches shaped like SURVEY §8(d)'s configs, plus edge cases.  Runs on a B200 (-m gpu)."""
from __future__ import annotations

import os
import random

import numpy as np
import pytest

from paper_conf_cluster_subdbn18_b200 import workloads as W
from tests.parity import compare

pytestmark = pytest.mark.gpu

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")
SMALL = dict(slots=148 * 128, heap_nodes=1 << 24, vstack_entries=2048)


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


def run_both(culi, oracle_mod, defs, forms, ctx_kw=None, oracle_kw=None):
    ctx = culi.Context(**{**SMALL, **(ctx_kw or {})})
    if defs:
        ctx.define(defs)
    res = ctx.eval_batch(forms)
    s = oracle_mod.Session(**(oracle_kw or {}))
    if defs:
        s.define(defs)
    o = s.eval_batch(forms, nthreads=os.cpu_count() or 1).results
    return res.printed(), res.steps(), o


def assert_parity(culi, oracle_mod, defs, forms, **kw):
    gp, gs, o = run_both(culi, oracle_mod, defs, forms, **kw)
    bad = compare(gp, gs, o, forms.splitlines())
    assert not bad, "\n".join(bad)
    return gp, gs, o


def _tsv(name):
    rows = []
    for line in open(os.path.join(GOLDEN, name)):
        if line.strip() and not line.startswith("#"):
            rows.append(line.rstrip("\n").split("\t"))
    return rows


DEFS = "\n".join([W.FIB_DEF, W.FACT_DEF, W.SUM_DEF, W.WHEN_DEF])


def test_paper_examples_and_step_pins(culi, oracle_mod):
    rows = _tsv("paper_examples.tsv") + _tsv("step_pins.tsv")
    forms = "\n".join(r[0] for r in rows)
    gp, gs, _ = assert_parity(culi, oracle_mod, DEFS, forms)
    for (f, exp, steps, *_), p, s in zip(rows, gp, gs):       # and the cited expected values directly
        assert (p, s) == (exp, int(steps)), f


def test_edge_cases(culi, oracle_mod):
    rows = _tsv("edge_cases.tsv")
    forms = "\n".join(r[0] for r in rows)
    gp, _, _ = assert_parity(culi, oracle_mod, DEFS, forms)
    assert gp == [r[1] for r in rows]


def test_empty_batch(culi):
    ctx = culi.Context(**SMALL)
    res = ctx.eval_batch("")
    assert len(res) == 0
    res = ctx.eval_batch("; only a comment\n")
    assert len(res) == 0


def test_parse_error(culi):
    ctx = culi.Context(**SMALL)
    with pytest.raises(culi.ParseError) as ei:
        ctx.read("(+ 1 2")
    assert ei.value.offset == 0


def test_c1_full(culi, oracle_mod):
    wl = W.c1()
    assert_parity(culi, oracle_mod, wl.defs, wl.forms)


def test_c2_small_full(culi, oracle_mod):
    wl = W.c2(3000, lo=0, hi=16)
    assert_parity(culi, oracle_mod, wl.defs, wl.forms)


def fib_py(n):
    a, b = 0, 1
    for _ in range(n):
        a, b = b, a + b
    return a


def test_c2_full_size(culi, oracle_mod):
    """configs[1] at full size in the bench's launch configuration (default Context): every form checked
    against the oracle's closed forms (pinned in test_oracle_pins), and a sample against the oracle."""
    wl = W.c2()
    ctx = culi.Context()
    ctx.define(wl.defs)
    res = ctx.eval_batch(wl.forms)
    lines = wl.form_lines()
    gp, gs = res.printed(), res.steps()
    for line, p, s in zip(lines, gp, gs):
        n = int(line[5:-1])
        assert p == str(fib_py(n)) and s == 27 * fib_py(n + 1) - 17, line
    s = oracle_mod.Session()
    s.define(wl.defs)
    rnd = random.Random(0)
    idx = sorted(rnd.sample(range(len(lines)), 48))
    o = s.eval("\n".join(lines[i] for i in idx))
    bad = compare([gp[i] for i in idx], [gs[i] for i in idx], o)
    assert not bad, bad


def test_c3_small(culi, oracle_mod):
    wl = W.c3(5000)
    assert_parity(culi, oracle_mod, wl.defs, wl.forms)


def test_c3_full(culi, oracle_mod):
    wl = W.c3()
    assert_parity(culi, oracle_mod, wl.defs, wl.forms, ctx_kw=dict(heap_nodes=1 << 26))
    ctx = culi.Context(**{**SMALL, "heap_nodes": 1 << 26})
    ctx.define(wl.defs)
    ctx.eval_batch(wl.forms)
    assert ctx.last_stats() == (1, 0)                 # the ||| form fanned out, no fallback


def test_c4_full(culi, oracle_mod):
    wl = W.c4()                                   # configs[3] at full size: 262,144 forms
    assert_parity(culi, oracle_mod, wl.defs, wl.forms, ctx_kw=dict(heap_nodes=1 << 27))


def test_c5_small(culi, oracle_mod):
    wl = W.c5(20000)
    assert_parity(culi, oracle_mod, wl.defs, wl.forms)


def test_c5_large(culi, oracle_mod):
    wl = W.c5(1 << 18)                            # 262,144 mixed forms, every one checked
    assert_parity(culi, oracle_mod, wl.defs, wl.forms, ctx_kw=dict(heap_nodes=1 << 27))


def test_c5_full_size(culi, oracle_mod):
    """configs[4] at full size (16,777,216 forms) in the bench's launch configuration, read on the device
    (the e2e path): every (fib n) / (fact n) form against its closed form (value and step count, pinned in
    test_oracle_pins), and a sample of every kind against the oracle."""
    import math
    wl = W.c5()
    ctx = culi.Context(heap_nodes=1 << 30)
    ctx.define(wl.defs)
    res = ctx.eval_text(wl.forms)
    lines = wl.form_lines()
    assert len(res) == len(lines) == 16777216
    _, nerr = res.totals()
    idx_closed = [i for i in range(0, len(lines), 997) if lines[i].startswith(("(fib ", "(fact "))]
    for i in idx_closed:
        t, e, st = res.info(i)
        n = int(lines[i].split()[1][:-1])
        if lines[i].startswith("(fib "):
            assert (res.int_value(i), st) == (fib_py(n), 27 * fib_py(n + 1) - 17), lines[i]
        else:
            w = (math.factorial(n) + 2 ** 63) % 2 ** 64 - 2 ** 63
            assert (res.int_value(i), st) == (w, 15 * n - 5 if n >= 2 else 10), lines[i]
    s = oracle_mod.Session()
    s.define(wl.defs)
    rnd = random.Random(7)
    idx = sorted(rnd.sample(range(len(lines)), 3000))
    o = s.eval("\n".join(lines[i] for i in idx))
    bad = compare([res.print(i) for i in idx], [res.info(i)[2] for i in idx], o)
    assert not bad, bad


def test_c0(culi, oracle_mod):
    for n in (1, 31, 32, 33, 1000, 4096):
        wl = W.c0(n)
        assert_parity(culi, oracle_mod, wl.defs, wl.forms)


def test_depth_and_fuel_limits(culi, oracle_mod):
    forms = "\n".join(["(sum %d)" % n for n in (10, 339, 340, 341, 400)] + ["(fib 12)", "(fact 30)"])
    assert_parity(culi, oracle_mod, DEFS, forms)
    assert_parity(culi, oracle_mod, DEFS, forms, ctx_kw=dict(max_depth=100, fuel=2000),
                  oracle_kw=dict(max_depth=100, fuel=2000))


def test_flags_do_not_change_results(culi, oracle_mod):
    wl = W.c5(5000)                      # above BIN_MIN_FORMS: the default run is binned
    outs = []
    for fl in (0, culi.CULI_F_NO_BINNING, culi.CULI_F_NO_VOTING | culi.CULI_F_NO_STAGING):
        gp, gs, o = run_both(culi, oracle_mod, wl.defs, wl.forms, ctx_kw=dict(flags=fl))
        outs.append((gp, gs))
        assert not compare(gp, gs, o)
    assert outs[0] == outs[1] == outs[2]


def test_global_persistence_and_redefine(culi):
    ctx = culi.Context(**SMALL)
    ctx.define("(define k 1) (define g (lambda (x) (+ x k)))")
    assert ctx.eval_batch("(g 10)").printed() == ["11"]
    ctx.define("(define k 5)")
    assert ctx.eval_batch("(g 10)").printed() == ["15"]


def test_define_failure(culi):
    ctx = culi.Context(**SMALL)
    with pytest.raises(culi.CuliError) as ei:
        ctx.define("(define a 1) (define b (/ 1 0)) (define c 3)")
    assert ei.value.failed_index == 1
    assert ctx.eval_batch("a\nb\nc").printed() == ["1", "b", "c"]


def test_closures_capturing_stack_frames(culi, oracle_mod):
    defs = """(define adder (lambda (k) (lambda (x) (+ x k))))
(define compose (lambda (f g) (lambda (x) (f (g x)))))
(define twice (lambda (f) (compose f f)))
(defmacro swap-args (f a b) (list f b a))"""
    forms = """((adder 3) 4)
(((twice (adder 5))) 1)
((twice (adder 5)) 1)
(let ((a 1)) (let ((f (lambda (y) (+ a y)))) (f 10)))
(let ((a 1) (b 2)) ((lambda () (let ((c 3)) ((lambda (d) (list a b c d)) 4)))))
(||| 3 (adder 10) '(1 2 3))
(||| 2 (lambda (x y) (let ((z (* x y))) (list x y z))) '(1 2) '(3 4))
(swap-args - 1 10)
(let ((f (lambda (n) (* n n)))) (||| 4 f '(1 2 3 4)))
(((lambda (a) (lambda (b) (lambda (c) (list a b c)))) 1) 2)
((((lambda (a) (lambda (b) (lambda (c) (list a b c)))) 1) 2) 3)"""
    assert_parity(culi, oracle_mod, defs, forms)


def test_random_programs(culi, oracle_mod):
    """Randomly generated nested programs over the whole language (fuzz parity)."""
    rnd = random.Random(1234)
    syms = ["x", "y", "z"]

    def expr(d):
        k = rnd.randint(0, 14 if d < 4 else 3)
        if k == 0:
            return str(rnd.randint(-20, 20))
        if k == 1:
            return repr(rnd.uniform(-5, 5))
        if k == 2:
            return rnd.choice(syms)
        if k == 3:
            return rnd.choice(["nil", "T", "'a", "'(1 2)"])
        if k == 4:
            return "(%s %s %s)" % (rnd.choice("+-*/"), expr(d + 1), expr(d + 1))
        if k == 5:
            return "(if %s %s %s)" % (expr(d + 1), expr(d + 1), expr(d + 1))
        if k == 6:
            return "(let ((%s %s)) %s)" % (rnd.choice(syms), expr(d + 1), expr(d + 1))
        if k == 7:
            return "((lambda (%s) %s) %s)" % (rnd.choice(syms), expr(d + 1), expr(d + 1))
        if k == 8:
            return "(list %s %s)" % (expr(d + 1), expr(d + 1))
        if k == 9:
            return "(%s %s)" % (rnd.choice(["car", "cdr", "length", "reverse", "null", "atom"]), expr(d + 1))
        if k == 10:
            return "(cons %s %s)" % (expr(d + 1), expr(d + 1))
        if k == 11:
            return "(%s %s %s)" % (rnd.choice(["<", "=", ">=", "eq", "equal", "rem", "mod", "nth"]),
                                   expr(d + 1), expr(d + 1))
        if k == 12:
            return "(when %s %s)" % (expr(d + 1), expr(d + 1))
        if k == 13:
            return "(append %s %s)" % (expr(d + 1), expr(d + 1))
        return "(||| 2 %s '(1 2) '(3 4))" % rnd.choice(["+", "list", "(lambda (a b) (* a b))", "cons"])

    forms = "\n".join(expr(0) for _ in range(4000))
    assert_parity(culi, oracle_mod, DEFS, forms)


def test_upload_eval_fetch_repeatable(culi, oracle_mod):
    wl = W.c5(2000)
    ctx = culi.Context(**SMALL)
    ctx.define(wl.defs)
    h = ctx.upload(wl.forms)
    for _ in range(3):
        ctx.eval_uploaded(h)
    r = ctx.fetch_results(h)
    s = oracle_mod.Session()
    s.define(wl.defs)
    assert not compare(r.printed(), r.steps(), s.eval(wl.forms))
    ms, kernels, high = ctx.last_timing()
    assert kernels >= 2 and all(m >= 0 for m in ms)
    ctx.release(h)


@pytest.mark.parametrize("cfg", ["c1", "c3", "c5"])
def test_graph_replay_on_a_stream(culi, oracle_mod, cfg):
    """culi_eval_uploaded on a non-default stream captures the device step into a CUDA graph and replays
    it: same results as direct launches (CULI_F_NO_GRAPH) and the oracle."""
    import torch
    wl = {"c1": lambda: W.c1(), "c3": lambda: W.c3(3000), "c5": lambda: W.c5(4000)}[cfg]()
    s = torch.cuda.Stream()
    out = []
    for flags in (0, culi.CULI_F_NO_GRAPH):
        ctx = culi.Context(**SMALL, stream=s.cuda_stream, flags=flags)
        if wl.defs:
            ctx.define(wl.defs)
        h = ctx.upload(wl.forms)
        for _ in range(4):
            ctx.eval_uploaded(h)
        r = ctx.fetch_results(h)
        out.append((r.printed(), r.steps()))
        ctx.eval_uploaded(h)                    # a replay after a fetch is still valid
        r2 = ctx.fetch_results(h)
        assert (r2.printed(), r2.steps()) == out[-1]
        ctx.release(h)
        ctx.close()
    assert out[0] == out[1]
    o = oracle_mod.Session()
    if wl.defs:
        o.define(wl.defs)
    assert not compare(out[0][0], out[0][1], o.eval(wl.forms))


def test_wide_forms(culi, oracle_mod):
    """Top-level forms with >= 64 arguments take the wide path (arguments one per thread, K12)."""
    rnd = random.Random(77)
    forms = []
    for n in (64, 65, 100, 257, 1000):
        forms.append("(list %s)" % " ".join(str(rnd.randint(-9, 9)) for _ in range(n)))
        forms.append("(+ %s)" % " ".join(str(rnd.randint(-2**62, 2**62)) for _ in range(n)))
        forms.append("(* %s)" % " ".join(str(rnd.randint(-3, 3)) for _ in range(n)))
        forms.append("(+ %s)" % " ".join(repr(rnd.uniform(-1e3, 1e3)) if rnd.random() < 0.5 else str(rnd.randint(-9, 9))
                                         for _ in range(n)))       # mixed int/float: sequential left fold
        forms.append("(%d %s)" % (n, " ".join("(fib %d)" % rnd.randint(0, 12) for _ in range(n))))
        forms.append("(foo %s)" % " ".join(rnd.choice(["x", "'y", "(fact 5)", "nil", "T", "\"s\""]) for _ in range(n)))
        forms.append("(list %s)" % " ".join("(list %d (+ %d 1))" % (i, i) for i in range(n)))
    forms.append("(list %s (car 5) %s)" % (" ".join(["1"] * 40), " ".join(["(fib 10)"] * 40)))   # error mid-way
    forms.append("(+ %s 'a %s)" % (" ".join(["1"] * 40), " ".join(["2"] * 40)))                    # TYPE after all args
    forms.append("(list %s)" % " ".join(["(sum 400)"] * 70))                                       # DEPTH inside
    text = "\n".join(forms)
    assert_parity(culi, oracle_mod, DEFS, text)
    ctx = culi.Context(**SMALL)
    ctx.define(DEFS)
    ctx.eval_batch(text)
    fan, fb = ctx.last_stats()
    assert fan == 5 * 7 + 3 and fb == 2, (fan, fb)    # every form above is wide (data/list/fold);
    # (foo ...) wide forms too; the mid-way error and the DEPTH form fall back, the TYPE fold does not


def test_wide_forms_fuel(culi, oracle_mod):
    forms = "(list %s)" % " ".join(["(fib 8)"] * 100)
    for fuel in (500, 6000, 6800, 100000):
        assert_parity(culi, oracle_mod, DEFS, forms, ctx_kw=dict(fuel=fuel), oracle_kw=dict(fuel=fuel))


NESTED_DEFS = "\n".join([W.FIB_DEF, W.FACT_DEF,
    "(define pfib (lambda (xs) (||| (length xs) fib xs)))",
    "(define psq (lambda (xs) (||| (length xs) (lambda (x) (* x x)) xs)))",
    "(define pscale (lambda (k xs) (||| (length xs) (lambda (x) (+ (* k x) 0.5)) xs)))",
    "(define xs40 '(%s))" % " ".join(str(i % 13) for i in range(40)),
    "(define xs100 '(%s))" % " ".join(str(i) for i in range(100)),
    "(define xs3000 '(%s))" % " ".join(str(i % 17) for i in range(3000))])


def test_nested_par(culi, oracle_mod):
    """||| below the top level: suspended evaluations resume with the elements' results."""
    forms = ["(pfib xs40)", "(car (pfib xs40))", "(+ 1 (length (psq xs100)))", "(psq xs3000)",
             "(pscale 3 xs100)", "(pscale 2.5 xs3000)", "(list (pfib xs40) (psq xs100))",
             "(let ((r (pfib xs40))) (equal r (pfib xs40)))",
             "(||| 2 pfib (list xs40 xs40))",                               # nested inside a top-level fan-out
             "(psq (list 1 2 3))",                                          # below NEST_MIN: sequential
             "(psq (cons 'a xs40))",                                        # element TYPE error -> fallback
             "(fact (length (psq xs100)))"] * 3
    text = "\n".join(forms)
    assert_parity(culi, oracle_mod, NESTED_DEFS, text)
    ctx = culi.Context(**SMALL)
    ctx.define(NESTED_DEFS)
    r = ctx.eval_batch(text)
    assert len(r) == len(forms)
    fan, fb = ctx.last_stats()
    # each call of pfib/psq/pscale on a >= 32-element list suspends once; the element-error form falls back
    assert ctx.last_nested >= 3 * 9 and fb >= 3, (fan, fb, ctx.last_nested)
    ctx2 = culi.Context(**SMALL, flags=culi.CULI_F_NO_NESTED)
    ctx2.define(NESTED_DEFS)
    r2 = ctx2.eval_batch(text)
    assert r.printed() == r2.printed() and r.steps() == r2.steps()


def test_nested_par_limits(culi, oracle_mod):
    forms = "\n".join(["(pfib xs40)", "(psq xs3000)", "(pscale 2 xs40)"])      # (fib <= 12) elements
    for fuel, depth in ((1 << 40, 1024), (5000, 1024), (200000, 1024), (1 << 40, 6), (1 << 40, 4)):
        assert_parity(culi, oracle_mod, NESTED_DEFS, forms, ctx_kw=dict(fuel=fuel, max_depth=depth),
                      oracle_kw=dict(fuel=fuel, max_depth=depth))


WIDE_DEFS = "\n".join([W.FIB_DEF, W.FACT_DEF,
    "(define wsq (lambda (k) (list %s)))" % " ".join("(* k %d)" % i for i in range(70)),
    "(define wdat (lambda (a b) (5 %s)))" % " ".join(("a", "b", "(+ a b)", "(fib a)", "'q", "2.5")[i % 6]
                                                     for i in range(90)),
    "(define wbad (lambda (a) (list %s)))" % " ".join(("(car a)" if i in (40, 60) else str(i)) for i in range(80)),
    "(define wq (lambda () '(%s)))" % " ".join(str(i) for i in range(100))])


def _wide(n, elem="5"):
    return "(%s)" % " ".join([elem] * n)


def test_wide_lists_below_top_level(culi, oracle_mod):
    """Wide data lists and (list a1..an) below the top level (>= WIDE_MIN elements): the
    evaluation suspends and any thread evaluates the elements (NEST_EVAL) — in a function body (stack
    environment, promoted to the heap), as a ||| argument (the paper-shaped C0), nested in each other, with
    element errors (exact sequential fallback: the first error in order) and under fuel/depth limits."""
    forms = ["(||| 100 fib %s)" % _wide(100), "(||| 64 fib %s)" % _wide(64), "(||| 63 fib %s)" % _wide(63),
             "(length (wsq 3))", "(wsq 7)", "(wdat 6 7)", "(car (cdr (wdat 10 2)))",
             "(wbad '(1 2))", "(wbad 5)", "(wq)", "(length (list %s))" % " ".join("(fib %d)" % (i % 15) for i in range(200)),
             "(list 1 %s 2)" % _wide(80, "(+ 1 2)"), "(+ 1 (length %s))" % _wide(300, "(fact 5)"),
             "(||| 3 + (1 2 3) (list %s))" % " ".join(str(i) for i in range(65)),
             "(let ((x 4)) (list %s))" % " ".join("(* x %d)" % i for i in range(66)),
             "(%s)" % " ".join(["(fib 10)"] * 65), "(1 %s)" % " ".join(["(undefined-f 1)"] * 70)] * 2
    text = "\n".join(forms)
    assert_parity(culi, oracle_mod, WIDE_DEFS, text)
    ctx = culi.Context(**SMALL)
    ctx.define(WIDE_DEFS)
    r = ctx.eval_batch(text)
    fan, fb = ctx.last_stats()
    assert ctx.last_nested >= 2 * 10 and fb >= 2, (fan, fb, ctx.last_nested)
    ctx2 = culi.Context(**SMALL, flags=culi.CULI_F_NO_NESTED)
    ctx2.define(WIDE_DEFS)
    r2 = ctx2.eval_batch(text)
    assert r.printed() == r2.printed() and r.steps() == r2.steps()
    # the same through the device reader (its RF_WIDE_NESTED flag selects the launch mode)
    ctx3 = culi.Context(**SMALL)
    ctx3.define_text(WIDE_DEFS)
    r3 = ctx3.eval_text(text)
    ctx3.last_stats()
    assert r3.printed() == r.printed() and r3.steps() == r.steps() and ctx3.last_nested >= 2 * 10
    for fuel, depth in ((3000, 1024), (1 << 40, 4), (1 << 40, 3)):
        assert_parity(culi, oracle_mod, WIDE_DEFS, text, ctx_kw=dict(fuel=fuel, max_depth=depth),
                      oracle_kw=dict(fuel=fuel, max_depth=depth))


def test_c0_paper_shape_full(culi, oracle_mod):
    """C0 at its bench size ((||| 4096 fib (5 5 ... 5))): the data list is evaluated by the
    whole grid, the elements fan out; value and steps equal the oracle's."""
    wl = W.c0(4096)
    assert_parity(culi, oracle_mod, wl.defs, wl.forms)
    ctx = culi.Context(**SMALL)
    ctx.define(wl.defs)
    ctx.eval_batch(wl.forms)
    ctx.last_stats()
    assert ctx.last_nested == 1


@pytest.mark.parametrize("n", [1, 2, 4095, 4096, 4097])
def test_small_batch_dispatch_boundary(culi, oracle_mod, n):
    """Batches of <= 4096 forms run in input order, larger ones through the binning permutation
    (BIN_MIN_FORMS, csrc/culi_eval.cuh): both must evaluate every form exactly once, in parity."""
    wl = W.c5(n, seed=77)
    gp, gs, o = assert_parity(culi, oracle_mod, wl.defs, wl.forms)
    ctx = culi.Context(**{**SMALL, "flags": culi.CULI_F_NO_BINNING})
    ctx.define(wl.defs)
    r = ctx.eval_batch(wl.forms)
    assert (r.printed(), r.steps()) == (gp, gs)


def test_no_closure_batch_runs_without_splitting(culi, oracle_mod):
    """Without lambda / defun anywhere (definitions or batch) no closure exists, so argument splitting is
    off and the grid shrinks (csrc/culi_capi.cu image_mentions_closure); a lambda turns it back on."""
    wl = W.c1()
    ctx = culi.Context(**SMALL)
    r = ctx.eval_batch(wl.forms)
    assert ctx.last_splits() == 0
    o = oracle_mod.Session().eval_batch(wl.forms, nthreads=os.cpu_count() or 1).results
    assert not compare(r.printed(), r.steps(), o, wl.forms.splitlines())
    fib = "(define fib (lambda (n) (if (< n 2) n (+ (fib (- n 1)) (fib (- n 2))))))"
    ctx.define(fib)
    r2 = ctx.eval_batch("(fib 22)\n" * 64)
    assert r2.printed() == ["17711"] * 64
    assert ctx.last_splits() > 0


@pytest.mark.timeout(600)
@pytest.mark.parametrize("flags", ["NO_BINNING", "binned"])
def test_unbinned_closure_batches_split(culi, oracle_mod, flags):
    """Regression (round 1: argument splitting on unbinned multi-form batches hung, so it was gated off):
    unbinned (diverged warps) and binned closure batches now split, repeatedly, in parity, and no bounded
    inter-warp wait ever gives up (atomic slot pick, ticket-stamped queue entries)."""
    wl = W.c5(2000)
    fl = culi.CULI_F_NO_BINNING if flags == "NO_BINNING" else 0
    ctx = culi.Context(**{**SMALL, "flags": fl})
    ctx.define(wl.defs)
    o = oracle_mod.Session()
    o.define(wl.defs)
    ores = o.eval(wl.forms)
    total = 0
    for _ in range(8):
        r = ctx.eval_batch(wl.forms)
        total += ctx.last_splits()
        assert ctx.last_waits()[0] == 0, ctx.last_waits()
        assert not compare(r.printed(), r.steps(), ores, wl.forms.splitlines())
    assert total > 0
    h = ctx.upload(wl.forms)                       # graph replay of the same unbinned step
    for _ in range(50):
        ctx.eval_uploaded(h)
    r = ctx.fetch_results(h)
    ctx.release(h)
    assert ctx.last_waits()[0] == 0
    assert not compare(r.printed(), r.steps(), ores, wl.forms.splitlines())


@pytest.mark.timeout(600)
def test_split_with_failing_forms_unbinned(culi, oracle_mod):
    """Forms that fail while split groups are pending (abandon_joins) mixed with recursive forms in the same
    warps, unbinned and repeated: parity, splits happen, no wait gives up."""
    defs = "\n".join([W.FIB_DEF, W.SUM_DEF])
    rng = np.random.default_rng(3)
    kinds = ["(+ (fib %d) (fib %d))", "(+ (fib %d) (car %d))", "(list (fib %d) (sum 400) %d)",
             "(+ (sum %d) (fib %d) (/ 1 0))", "(- (fib %d) (fib %d))"]
    forms = []
    for _ in range(3000):
        k = kinds[rng.integers(0, len(kinds))]
        forms.append(k % (rng.integers(8, 19), rng.integers(5, 16)))
    text = "\n".join(forms)
    gp, gs, o = run_both(culi, oracle_mod, defs, text, ctx_kw=dict(flags=culi.CULI_F_NO_BINNING))
    assert not compare(gp, gs, o, forms)
    ctx = culi.Context(**{**SMALL, "flags": culi.CULI_F_NO_BINNING})
    ctx.define(defs)
    splits = 0
    for _ in range(6):
        r = ctx.eval_batch(text)
        splits += ctx.last_splits()
        assert ctx.last_waits()[0] == 0, ctx.last_waits()
        assert (r.printed(), r.steps()) == (gp, gs)
    assert splits > 0


def test_define_while_uploaded_is_a_state_error(culi):
    """culi_define while a batch is uploaded would put definitions below the batch: CULI_E_STATE."""
    ctx = culi.Context(**SMALL)
    ctx.define(W.FIB_DEF)
    h = ctx.upload("(fib 10)")
    with pytest.raises(culi.CuliError) as ei:
        ctx.define("(define x 1)")
    assert ei.value.status == -7
    with pytest.raises(culi.CuliError):
        ctx.define_text("(define x 1)")
    ctx.release(h)
    ctx.define("(define x 1)")
    assert ctx.eval_batch("(+ x (fib 10))").printed() == ["56"]


DEFUN_DEFS = "\n".join([
    "(defun sq (x) (* x x))",
    "(defun k42 () 42)",
    "(defun two (x) (+ x 1) (* x 2))",
    "(defun fibd (n) (if (< n 2) n (+ (fibd (- n 1)) (fibd (- n 2)))))",
    "(defun factd (n) (if (< n 2) 1 (* n (factd (- n 1)))))",
    "(defun add3 (a b c) (+ a (* 10 b) (* 100 c)))",
    "(defun mk (k) (lambda (x) (+ x k)))",
])


def test_defun_definitions(culi, oracle_mod):
    """defun (SURVEY c.13 #12): functions defined with defun, through the host
    reader and the device reader, against the oracle and the closed forms pinned in test_oracle_pins."""
    forms = ["(sq 7)", "(k42)", "(two 5)", "(add3 1 2 3)", "sq", "(sq)", "(sq 'a)", "((mk 3) 4)",
             "(||| 4 sq '(1 2 3 4))", "(||| 3 (mk 10) '(1 2 3))", "(defun z (x) x)"]
    forms += ["(fibd %d)" % (n % 19) for n in range(600)] + ["(factd %d)" % (n % 22) for n in range(300)]
    text = "\n".join(forms)
    gp, gs, _ = assert_parity(culi, oracle_mod, DEFUN_DEFS, text)
    assert gp[:5] == ["49", "42", "10", "321", "#<lambda>"] and gs[:4] == [7, 3, 11, 16]
    assert gp[10] == "#<error DEFINE_IN_BATCH>"
    for f, p, s in zip(forms, gp, gs):
        if f.startswith("(fibd"):
            n = int(f[6:-1])
            assert (int(p), s) == (fib_py(n), 27 * fib_py(n + 1) - 17), f
    ctx = culi.Context(**SMALL)
    ctx.define_text(DEFUN_DEFS)
    r = ctx.eval_text(text)
    assert (r.printed(), r.steps()) == (gp, gs)
    # redefinition through defun is seen by existing callers (late binding, L447-448)
    ctx.define_text("(defun h (x) (sq (sq x)))")
    assert ctx.eval_batch("(h 3)").printed() == ["81"]
    ctx.define("(defun sq (x) (+ x x))")
    assert ctx.eval_batch("(h 3)").printed() == ["12"]


def test_quasiquote(culi, oracle_mod):
    """Quasiquote (reading R8): the hand-derived pins, random templates with unquote,
    unquote-splicing and nesting, and macros written with templates — host reader and device reader."""
    rows = _tsv("quasiquote_pins.tsv")
    rnd = random.Random(21)

    def tmpl(d):
        k = rnd.randint(0, 6 if d < 3 else 2)
        if k == 0:
            return str(rnd.randint(-9, 9))
        if k == 1:
            return rnd.choice(["a", "b", "nil", "T", '"s"', "2.5"])
        if k == 2:
            return ",(+ %d x)" % rnd.randint(-5, 5)
        if k == 3:
            return "(unquote-splicing (list %d x))" % rnd.randint(0, 3)
        if k == 4:
            return "`(q %s)" % tmpl(d + 1)
        if k == 5:
            return "(unquote-splicing %s)" % rnd.choice(["nil", "5", "'(1 2)", "(cons 1 2)"])
        return "(%s)" % " ".join(tmpl(d + 1) for _ in range(rnd.randint(0, 4)))

    forms = [r[0] for r in rows] + ["(let ((x %d)) `%s)" % (rnd.randint(-3, 3), tmpl(0)) for _ in range(600)]
    defs = "\n".join([
        "(defmacro my-if (c a b) `(if ,c ,a ,b))",
        "(defmacro swap (a b) `(list ,b ,a))",
        "(defmacro my-let1 (v e body) `((lambda (,v) ,body) ,e))",
        "(defmacro build (n) `(list (unquote-splicing (list n n)) ,n))",
        "(define k 7)"])
    forms += ["(my-if (< %d 0) 'neg 'nonneg)" % v for v in range(-3, 3)]
    forms += ["(swap 1 2)", "(my-let1 y (+ 1 2) (* y y))", "`(k ,k)", "(build 4)"]
    text = "\n".join(forms)
    gp, gs, _ = assert_parity(culi, oracle_mod, defs, text)
    for r, p, st in zip(rows, gp, gs):
        assert (p, st) == (r[1], int(r[2])), r
    ctx = culi.Context(**SMALL)
    ctx.define_text(defs)
    r = ctx.eval_text(text)
    assert (r.printed(), r.steps()) == (gp, gs)
