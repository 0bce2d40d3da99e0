"""Seeded synthetic program generators for configs C0-C5 (BASELINE.json `configs`).

This module only emits Lisp *text*; it holds none of the method's arithmetic.  It is the one module the
oracle side (tests, bench cpu_baseline) and the CUDA side (tests, bench) share.  Format (§8(d) "Text
format"): one top-level form per line, tokens separated by one space, no space after "(" or before ")",
decimal ints, floats printed with Python ``repr``.  Seeds are 1000 + config number.

Each generator returns ``Workload(name, defs, forms, nforms, units)`` where ``units`` is the number of
"forms" the forms/sec metric counts (top-level forms, or ||| element applications for C0/C3).
"""
from __future__ import annotations

import dataclasses
import hashlib
import os

import numpy as np

GEN_VERSION = 1

FIB_DEF = "(define fib (lambda (n) (if (< n 2) n (+ (fib (- n 1)) (fib (- n 2))))))"
FACT_DEF = "(define fact (lambda (n) (if (< n 2) 1 (* n (fact (- n 1))))))"
SUM_DEF = "(define sum (lambda (n) (if (= n 0) 0 (+ n (sum (- n 1))))))"
SUM_LIST_DEF = "(define sum-list (lambda (l) (if (null l) 0 (+ (car l) (sum-list (cdr l))))))"
WHEN_DEF = "(defmacro when (c x) (list 'if c x nil))"

C4_MACROS = [
    "(defmacro when (c x) (list 'if c x nil))",
    "(defmacro unless (c x) (list 'if c nil x))",
    "(defmacro my-and (a b) (list 'if a b nil))",
    "(defmacro my-or (a b) (list 'if a T b))",
    "(defmacro inc (x) (list '+ x 1))",
    "(defmacro dec (x) (list '- x 1))",
    "(defmacro square (x) (list '* x x))",
    "(defmacro cond3 (c1 e1 c2 e2 e3) (list 'if c1 e1 (list 'if c2 e2 e3)))",
]

C3_DEFS_HEAD = [
    "(define make-f (lambda (k) (lambda (x) (let ((y (* k x)) (z (+ x 1.5))) (/ (+ (* y y) z) 2.0)))))",
    "(define f (make-f 0.75))",
]


@dataclasses.dataclass
class Workload:
    name: str
    defs: str
    forms: str
    nforms: int          # top-level forms in `forms`
    units: int           # units counted by forms/sec (forms, or ||| element applications)
    seed: int

    def sha256(self) -> str:
        h = hashlib.sha256()
        h.update(self.defs.encode())
        h.update(b"\0")
        h.update(self.forms.encode())
        return h.hexdigest()

    def form_lines(self) -> list[str]:
        return self.forms.splitlines()


def _rng(seed: int) -> np.random.Generator:
    return np.random.Generator(np.random.PCG64(seed))


# ---- C0: paper-shaped ||| fib(5) per worker (Fig.15) -------------------------------
def c0(n: int = 4096, seed: int = 1000) -> Workload:
    forms = "(||| %d fib (%s))" % (n, " ".join(["5"] * n)) if n > 0 else "(||| 0 fib nil)"
    return Workload("C0", FIB_DEF, forms + "\n", 1, n, seed)


# ---- C1: independent integer arithmetic trees, op-depth <= 4 (BASELINE configs[0]) ----------------
def c1(n: int = 1024, seed: int = 1001) -> Workload:
    rng = _rng(seed)
    ops = ["+", "-", "*"]

    def gen(level: int, dmax: int) -> str:
        op = ops[int(rng.integers(0, 3))]
        kids = []
        for _ in range(2):
            if level < dmax and rng.random() < 0.7:
                kids.append(gen(level + 1, dmax))
            else:
                kids.append(str(int(rng.integers(-99, 100))))
        return "(%s %s %s)" % (op, kids[0], kids[1])

    lines = []
    for _ in range(n):
        d = int(rng.integers(1, 5))
        lines.append(gen(1, d))
    return Workload("C1", "", "\n".join(lines) + "\n", n, n, seed)


# ---- C2: (fib n), n in 15..22, via a defined recursive lambda (BASELINE configs[1]) --------------
def c2(n: int = 65536, seed: int = 1002, lo: int = 15, hi: int = 23) -> Workload:
    rng = _rng(seed)
    ns = rng.integers(lo, hi, size=n)
    forms = "\n".join("(fib %d)" % int(k) for k in ns) + "\n"
    return Workload("C2", FIB_DEF, forms, n, n, seed)


# ---- C3: ||| of a closure (closure + let + float arithmetic) over a 1M-element list --------------
def c3(n: int = 1 << 20, seed: int = 1003) -> Workload:
    rng = _rng(seed)
    xs = rng.uniform(-4.0, 4.0, size=n)
    xs_text = " ".join(repr(float(x)) for x in xs)
    defs = "\n".join(C3_DEFS_HEAD + ["(define xs '(%s))" % xs_text]) + "\n"
    forms = "(||| %d f xs)\n" % n
    return Workload("C3", defs, forms, 1, n, seed)


# ---- fast chunked drawing (C4, C5) ------------------------------------------------------------------
# Big batches are generated in chunks of CHUNK forms; chunk c draws from PCG64(SeedSequence(seed).spawn)
# [c], so the text is identical however many processes generate it.  Draws come from a pre-generated
# block of uniforms: integers(lo, hi) = lo + floor(u * (hi - lo)).
CHUNK = 1 << 15


class _Draw:
    def __init__(self, seq: np.random.SeedSequence):
        self.g = np.random.Generator(np.random.PCG64(seq))
        self.buf = self.g.random(1 << 16).tolist()
        self.i = 0

    def u(self) -> float:
        if self.i >= len(self.buf):
            self.buf = self.g.random(1 << 16).tolist()
            self.i = 0
        x = self.buf[self.i]
        self.i += 1
        return x

    def int(self, lo: int, hi: int) -> int:          # uniform in [lo, hi)
        return lo + int(self.u() * (hi - lo))


def _chunked(fn, n: int, seed: int, procs: int | None = None) -> list[str]:
    nchunks = (n + CHUNK - 1) // CHUNK
    seqs = np.random.SeedSequence(seed).spawn(max(nchunks, 1))
    jobs = [(fn, seqs[c], min(CHUNK, n - c * CHUNK)) for c in range(nchunks)]
    if nchunks <= 16 or procs == 1:
        parts = [_run_chunk(j) for j in jobs]
    else:                                             # spawn: the caller may hold CUDA / NCCL threads
        import multiprocessing as mp
        with mp.get_context("spawn").Pool(procs or min(16, os.cpu_count() or 1)) as pool:
            parts = pool.map(_run_chunk, jobs, chunksize=1)
    return [line for part in parts for line in part]


def _run_chunk(job):
    fn, seq, count = job
    r = _Draw(seq)
    return [fn(r) for _ in range(count)]


# ---- C4: macro-heavy control forms (BASELINE configs[3]) ------------------------------------------
def _c4_form(r: _Draw) -> str:
    def leaf() -> str:
        return str(r.int(-20, 21))

    def I(d: int) -> str:
        if d == 0:
            return leaf()
        u = r.u()
        if u < 0.35:
            return "(%s %s)" % (("inc", "dec", "square")[r.int(0, 3)], I(d - 1))
        if u < 0.60:
            op = "+-*"[r.int(0, 3)]
            a = I(d - 1)
            return "(%s %s %s)" % (op, a, I(d - 1))
        return leaf()

    def B(d: int) -> str:
        if d == 0:
            c = "<=>"[r.int(0, 3)]
            a = leaf()
            return "(%s %s %s)" % (c, a, leaf())
        if r.u() < 0.3:
            m = ("my-and", "my-or")[r.int(0, 2)]
            a = B(d - 1)
            return "(%s %s %s)" % (m, a, B(d - 1))
        c = "<=>"[r.int(0, 3)]
        a = I(d - 1)
        return "(%s %s %s)" % (c, a, I(d - 1))

    k = r.int(0, 5)
    if k == 0:
        b = B(2)
        return "(when %s %s)" % (b, I(2))
    if k == 1:
        b = B(2)
        return "(unless %s %s)" % (b, I(2))
    if k == 2:
        b1 = B(2); i1 = I(2); b2 = B(2); i2 = I(2); i3 = I(2)
        return "(cond3 %s %s %s %s %s)" % (b1, i1, b2, i2, i3)
    if k == 3:
        m = ("my-and", "my-or")[r.int(0, 2)]
        a = B(2)
        return "(%s %s %s)" % (m, a, B(2))
    return "(%s %s)" % (("inc", "dec", "square")[r.int(0, 3)], I(2))


def c4(n: int = 262144, seed: int = 1004, procs: int | None = None) -> Workload:
    lines = _chunked(_c4_form, n, seed, procs)
    return Workload("C4", "\n".join(C4_MACROS) + "\n", "\n".join(lines) + "\n", n, n, seed)


# ---- C5: 16M mixed forms (fib / fact / list ops), sharded over 1/2/4/8 GPUs --------------------------
def _c5_list(r: _Draw, d: int) -> str:
    if d == 0 or r.u() < 0.4:
        k = r.int(0, 9)
        return "(list%s)" % "".join(" %d" % r.int(-50, 51) for _ in range(k))
    c = r.int(0, 4)
    if c == 0:
        i = r.int(-50, 51)
        return "(cons %d %s)" % (i, _c5_list(r, d - 1))
    if c == 1:
        return "(cdr %s)" % _c5_list(r, d - 1)
    if c == 2:
        return "(reverse %s)" % _c5_list(r, d - 1)
    a = _c5_list(r, d - 1)
    return "(append %s %s)" % (a, _c5_list(r, d - 1))


def _c5_form(r: _Draw) -> str:
    kind = r.int(0, 3)
    if kind == 0:
        return "(fib %d)" % r.int(5, 16)
    if kind == 1:
        return "(fact %d)" % r.int(1, 21)
    root = r.int(0, 6)
    L = _c5_list(r, 2)
    if root == 0:
        return "(length %s)" % L
    if root == 1:
        return "(car %s)" % L
    if root == 2:
        return "(sum-list %s)" % L
    if root == 3:
        return "(nth %d %s)" % (r.int(0, 9), L)
    if root == 4:
        return L
    L2 = L if r.u() < 0.5 else _c5_list(r, 2)
    return "(equal %s %s)" % (L, L2)


def c5(n: int = 16777216, seed: int = 1005, procs: int | None = None) -> Workload:
    lines = _chunked(_c5_form, n, seed, procs)
    defs = "\n".join([FIB_DEF, FACT_DEF, SUM_LIST_DEF]) + "\n"
    return Workload("C5", defs, "\n".join(lines) + "\n", n, n, seed)


CONFIGS = {"C0": c0, "C1": c1, "C2": c2, "C3": c3, "C4": c4, "C5": c5}


def shard_lines(forms: str, rank: int, world: int) -> tuple[str, list[int]]:
    """Strided dealing of forms over ranks: rank r takes {i : i mod k = r}."""
    lines = forms.splitlines()
    idx = list(range(rank, len(lines), world))
    return "\n".join(lines[i] for i in idx) + ("\n" if idx else ""), idx
