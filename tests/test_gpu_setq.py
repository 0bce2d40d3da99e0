"""GPU parity of setq (§III-B.a; reading R7 and §5.8): the
hand-derived pins of tests/golden/setq_pins.tsv, random mutation programs against the oracle, sequential
||| with a shared accumulator, define-time mutation, and batches that only inherit setq from definitions."""
from __future__ import annotations

import os
import random

import pytest

from paper_conf_cluster_subdbn18_b200 import workloads as W
from tests.parity import compare
from tests.test_oracle_pins import SETQ_DEFS

pytestmark = pytest.mark.gpu

SMALL = dict(slots=148 * 128, heap_nodes=1 << 24, vstack_entries=2048)
GOLDEN = os.path.join(os.path.dirname(__file__), "golden")


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


def _rows():
    return [l.rstrip("\n").split("\t") for l in open(os.path.join(GOLDEN, "setq_pins.tsv"))
            if l.strip() and not l.startswith("#")]


@pytest.mark.parametrize("device_read", [False, True])
def test_setq_pins(culi, oracle_mod, device_read):
    rows = _rows()
    forms = "\n".join(r[0] for r in rows)
    ctx = culi.Context(**SMALL)
    if device_read:
        ctx.define_text(SETQ_DEFS)
        res = ctx.eval_text(forms)
    else:
        ctx.define(SETQ_DEFS)
        res = ctx.eval_batch(forms)
    assert [(p, s) for p, s in zip(res.printed(), res.steps())] == [(r[1], int(r[2])) for r in rows]
    s = oracle_mod.Session()
    s.define(SETQ_DEFS)
    assert not compare(res.printed(), res.steps(), s.eval(forms))


def _rand_prog(r: random.Random) -> str:
    k = r.randint(1, 6)
    xs = " ".join(str(r.randint(-9, 9)) for _ in range(k))
    pick = r.randrange(6)
    if pick == 0:                                      # accumulate over a list with a sequential |||
        return "(let ((acc %d)) (||| %d (lambda (x) (setq acc (%s acc x))) '(%s)) acc)" % (
            r.randint(-5, 5), k, r.choice(["+", "-", "*"]), xs)
    if pick == 1:                                      # counters
        return "(let ((c (make-counter))) %s)" % " ".join(["(c)"] * r.randint(1, 9))
    if pick == 2:                                      # shadowing and the outer binding
        return "(let ((x %d)) (let ((x %d)) (setq x (* x 2)) x) (setq x (+ x 1)) x)" % (
            r.randint(-50, 50), r.randint(-50, 50))
    if pick == 3:                                      # recursion that mutates a captured variable
        return ("(let ((n 0)) (let ((f (lambda (self k) (if (< k 1) n (progn (setq n (+ n k)) (self self (- k 1)))))))"
                " (f f %d)))" % r.randint(0, 30))
    if pick == 4:                                      # errors: batch setq of globals / define-time frames
        return r.choice(["(setq g 1)", "(counter)", "(let ((x 1)) (setq x (car x)) x)", "(setq)"])
    return "(fib %d)" % r.randint(0, 12)               # forms without setq in the same batch


def test_random_setq_programs(culi, oracle_mod):
    r = random.Random(21)
    defs = SETQ_DEFS + "\n" + W.FIB_DEF
    forms = "\n".join(_rand_prog(r) for _ in range(3000))
    for reader in ("host", "device"):
        ctx = culi.Context(**SMALL)
        if reader == "host":
            ctx.define(defs)
            res = ctx.eval_batch(forms)
        else:
            ctx.define_text(defs)
            res = ctx.eval_text(forms)
        s = oracle_mod.Session()
        s.define(defs)
        bad = compare(res.printed(), res.steps(), s.eval_batch(forms, nthreads=os.cpu_count() or 1).results,
                      forms.splitlines())
        assert not bad, "\n".join(bad)


def test_inherited_setq_and_plain_batches(culi, oracle_mod):
    """A batch with no setq of its own still calls setq-using closures from the definitions; a session
    without setq anywhere keeps the fan-out path."""
    ctx = culi.Context(**SMALL)
    ctx.define(SETQ_DEFS + "\n(define bump (lambda (l) (let ((s 0)) (||| 40 (lambda (x) (setq s (+ s x))) l) s)))")
    xs = " ".join(str(i) for i in range(40))
    res = ctx.eval_batch("(bump '(%s))\n(let ((c (make-counter))) (c) (c))\nk1" % xs)
    assert res.printed() == [str(sum(range(40))), "2", "1"]
    plain = culi.Context(**SMALL)
    plain.define(W.FIB_DEF)
    r = plain.eval_batch("(||| 40 fib '(%s))" % " ".join(["7"] * 40))
    assert plain.last_stats() == (1, 0) and r.printed() == ["(%s)" % " ".join(["13"] * 40)]


def test_define_time_setq_and_reclamation(culi, oracle_mod):
    defs = "(define a 1)\n(setq a (+ a 41))\n(setq fresh 'made)\n(define f (lambda () a))\n" + SETQ_DEFS
    ctx = culi.Context(**SMALL)
    ctx.define_text(defs)
    ctx.collect()
    res = ctx.eval_batch("a\nfresh\n(f)\nk1\nk2\n(counter)")
    s = oracle_mod.Session()
    s.define(defs)
    assert not compare(res.printed(), res.steps(), s.eval("a\nfresh\n(f)\nk1\nk2\n(counter)"))
    assert res.printed()[:5] == ["42", "made", "42", "1", "2"]
