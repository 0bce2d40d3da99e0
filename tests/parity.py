"""Parity predicate between the CUDA path and the oracle.  Test infrastructure.

Two printed results agree when their token streams agree: same error name; same structure; INT /
SYMBOL / STRING tokens byte-equal; FLOAT tokens within |g - o| <= 1e-12 * max(|g|, |o|) (north_star's
tolerance; expected bit-exact under c.9), both nan, or equal infinities; and the canonical step counts are
equal.
"""
from __future__ import annotations

import math
import re

FLOAT_TOL = 1e-12
_TOK = re.compile(r'"[^"]*"|\(|\)|[^\s()]+')
_FLOAT = re.compile(r"^[+-]?(\d+\.\d*|\.\d+)([eE][+-]?\d+)?$|^[+-]?\d+[eE][+-]?\d+$|^-?inf$|^nan$")


def _ftok(t: str):
    if _FLOAT.match(t):
        return float(t)
    return None


def same_printed(g: str, o: str) -> bool:
    if g == o:
        return True
    tg, to = _TOK.findall(g), _TOK.findall(o)
    if len(tg) != len(to):
        return False
    for a, b in zip(tg, to):
        if a == b:
            continue
        fa, fb = _ftok(a), _ftok(b)
        if fa is None or fb is None:
            return False
        if math.isnan(fa) and math.isnan(fb):
            continue
        if math.isinf(fa) or math.isinf(fb):
            if fa != fb:
                return False
            continue
        if abs(fa - fb) > FLOAT_TOL * max(abs(fa), abs(fb)):
            return False
    return True


def compare(gpu_printed, gpu_steps, oracle_results, forms=None, max_report=5):
    """Return a list of human-readable mismatches (empty = parity)."""
    bad = []
    assert len(gpu_printed) == len(oracle_results), (len(gpu_printed), len(oracle_results))
    for i, (gp, gs, o) in enumerate(zip(gpu_printed, gpu_steps, oracle_results)):
        if o.err == 9:        # OOM is a resource error, never parity-checked (c.10)
            continue
        if not same_printed(gp, o.printed) or gs != o.steps:
            f = forms[i] if forms else ""
            bad.append("form %d %s: gpu=(%s, %d) oracle=(%s, %d)" % (i, f[:80], gp[:120], gs,
                                                                    o.printed[:120], o.steps))
            if len(bad) >= max_report:
                break
    return bad
