"""GPU parity of argument splitting: idle warps evaluate pending arguments split off busy
warps.  Arguments are pure inside a batch (SURVEY c.3, c.13 #25), so results must equal the oracle's —
value, canonical steps (c.4), the first error in evaluation order and the fuel limit (c.10) — whether an
argument was split off or not.  Batches here are small on a full grid, so idle warps exist and splits
happen (asserted through culi_last_splits)."""
from __future__ import annotations

import numpy as np
import pytest

from paper_conf_cluster_subdbn18_b200 import workloads as W
from tests.test_gpu_parity import SMALL, assert_parity, culi  # noqa: F401  (fixture)

pytestmark = pytest.mark.gpu

DEFS = "\n".join([W.FIB_DEF, W.FACT_DEF, W.SUM_DEF, W.WHEN_DEF,
                  "(define tree (lambda (n) (if (< n 1) 'leaf (list n (tree (- n 1)) (tree (- n 2))))))",
                  "(define fsum (lambda (n) (if (< n 2) 1.5 (+ (fsum (- n 1)) (* 0.5 (fsum (- n 2)))))))",
                  "(define pick (lambda (a b c) (if (< a b) c (+ a b c))))"])


def _ctx(culi, **kw):
    return culi.Context(**{**SMALL, **kw})


def _run(culi, text, **kw):
    ctx = _ctx(culi, **kw)
    ctx.define(DEFS)
    r = ctx.eval_batch(text)
    return r.printed(), r.steps(), ctx.last_splits()


def test_split_fib_batch(culi, oracle_mod):
    rng = np.random.default_rng(7)
    forms = ["(fib %d)" % n for n in rng.integers(14, 21, 200)] + ["(fib 22)"] * 40
    text = "\n".join(forms)
    assert_parity(culi, oracle_mod, DEFS, text)
    gp, gs, splits = _run(culi, text)
    assert splits > 0
    gp2, gs2, splits2 = _run(culi, text, flags=culi.CULI_F_NO_SPLIT)
    assert splits2 == 0 and (gp, gs) == (gp2, gs2)


def test_split_values_of_every_kind(culi, oracle_mod):
    """split-off arguments returning lists, floats, closures and symbols; 3+ arguments; closures calls"""
    forms = ["(length (tree 14))", "(car (cdr (tree 13)))", "(fsum 19)", "(pick (fib 18) (fib 17) (fib 16))",
             "(pick (fib 16) (fib 18) (list (fib 15) 'x))", "(list (fib 17) (fsum 15) (tree 3) 'done)",
             "(equal (tree 12) (tree 12))", "((lambda (a b) (- a b)) (fib 19) (fib 18))",
             "(let ((a (fib 18)) (b (fib 17))) (+ a b))", "(when (< (fib 17) (fib 18)) (fib 16))"]
    text = "\n".join(f for f in forms for _ in range(32))
    assert_parity(culi, oracle_mod, DEFS, text)
    _, _, splits = _run(culi, text)
    assert splits > 0


def test_split_errors_first_in_order(culi, oracle_mod):
    """an error in a split-off argument, in the argument before it, or in both: the first one wins"""
    forms = ["(+ (fib 18) (car 5))", "(+ (fib 18) (/ 1 0))", "(+ (car 5) (fib 18))",
             "(+ (fib 18) (fib 17) (rem 1 0))", "(+ (fib 17) (sum 400))", "(+ (sum 400) (fib 17) (car 1))",
             "(list (fib 18) (fib 16) (+ 'a 1))", "(pick (fib 18) (fact 5) (foo (car 3)))",
             "(+ (fib 18) (+ (fib 12) (car 2)))"]
    text = "\n".join(f for f in forms for _ in range(32))
    assert_parity(culi, oracle_mod, DEFS, text)
    _, _, splits = _run(culi, text)
    assert splits > 0


@pytest.mark.parametrize("fuel", [10, 60000, 112871, 112873, 130000, 182622, 182623, 182624, 1 << 40])
def test_split_fuel_limit(culi, oracle_mod, fuel):
    """fuel runs out before, inside or exactly at the end of a split-off argument (c.10)"""
    # (+ (fib 18) (fib 17)): 2 + S(18) + S(17) = 2 + 112,870 + 69,751 = 182,623 steps
    text = "\n".join(["(+ (fib 18) (fib 17))"] * 64 + ["(+ (fib 18) (fib 17) (car 1))"] * 32)
    assert_parity(culi, oracle_mod, DEFS, text, ctx_kw=dict(fuel=fuel), oracle_kw=dict(fuel=fuel))


@pytest.mark.parametrize("depth", [20, 24, 40])
def test_split_depth_limit(culi, oracle_mod, depth):
    text = "\n".join(["(+ (fib 18) (sum 8))", "(+ (fib 17) (sum 12))", "(+ (fib 18) (fib 17))"] * 32)
    assert_parity(culi, oracle_mod, DEFS, text, ctx_kw=dict(max_depth=depth),
                  oracle_kw=dict(max_depth=depth))
