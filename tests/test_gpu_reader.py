"""GPU parity of the device reader (culi_define_text / culi_eval_text / culi_upload_text):
program text read ON THE DEVICE must give, form by form, the oracle's printed values and step counts
(SURVEY §8(c).11), and the host reader's error offsets.  Float literals are additionally pinned to Python's
correctly rounded float() (an implementation independent of both the oracle's strtod and the device's
Eisel-Lemire + big-integer path), bit for bit, including halfway cases and > 780-digit inputs."""
from __future__ import annotations

import os
import random
import struct
from fractions import Fraction

import pytest

from paper_conf_cluster_subdbn18_b200 import workloads as W
from tests.parity import compare

pytestmark = pytest.mark.gpu

SMALL = dict(slots=148 * 128, heap_nodes=1 << 24, vstack_entries=2048)
DEFS = "\n".join([W.FIB_DEF, W.FACT_DEF, W.SUM_DEF, W.SUM_LIST_DEF, W.WHEN_DEF])
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


def text_parity(culi, oracle_mod, defs, forms, ctx_kw=None, device_defs=True):
    ctx = culi.Context(**{**SMALL, **(ctx_kw or {})})
    if defs:
        (ctx.define_text if device_defs else ctx.define)(defs)
    res = ctx.eval_text(forms)
    s = oracle_mod.Session()
    if defs:
        s.define(defs)
    o = s.eval_batch(forms, nthreads=os.cpu_count() or 1).results
    bad = compare(res.printed(), res.steps(), o, forms.splitlines())
    assert not bad, "\n".join(bad)
    return ctx, res


def _tsv(name):
    rows = []
    for line in open(os.path.join(GOLDEN, name)):
        if line.strip() and not line.startswith("#"):
            rows.append(line.rstrip("\n").split("\t"))
    return rows


def test_pins_and_edge_cases(culi, oracle_mod):
    rows = _tsv("paper_examples.tsv") + _tsv("step_pins.tsv") + _tsv("edge_cases.tsv")
    text_parity(culi, oracle_mod, DEFS, "\n".join(r[0] for r in rows))


@pytest.mark.parametrize("cfg", ["c1", "c2", "c4", "c5"])
def test_configs_small(culi, oracle_mod, cfg):
    wl = {"c1": lambda: W.c1(), "c2": lambda: W.c2(2000, lo=0, hi=16), "c4": lambda: W.c4(6000),
          "c5": lambda: W.c5(20000)}[cfg]()
    text_parity(culi, oracle_mod, wl.defs, wl.forms, ctx_kw=dict(heap_nodes=1 << 26))


def test_c3_full_device_read(culi, oracle_mod):
    """configs[2] at full size: the 1M-float definition and the ||| form both read on the device."""
    wl = W.c3()
    ctx, res = text_parity(culi, oracle_mod, wl.defs, wl.forms, ctx_kw=dict(heap_nodes=1 << 26))
    assert ctx.last_stats() == (1, 0)                  # the ||| form still fans out


def test_c5_large_same_as_host_reader(culi, oracle_mod):
    wl = W.c5(1 << 17)
    ctx = culi.Context(**{**SMALL, "heap_nodes": 1 << 27})
    ctx.define_text(wl.defs)
    a = ctx.eval_text(wl.forms)
    b = ctx.eval_batch(wl.forms)
    assert a.printed() == b.printed() and a.steps() == b.steps()
    ms, items, nodes = ctx.last_read()
    assert items > 0 and nodes > 0 and ms > 0
    s = oracle_mod.Session()
    s.define(wl.defs)
    lines = wl.form_lines()
    idx = sorted(random.Random(5).sample(range(len(lines)), 400))
    o = s.eval("\n".join(lines[i] for i in idx))
    ap, ast = a.printed(), a.steps()
    bad = compare([ap[i] for i in idx], [ast[i] for i in idx], o)
    assert not bad, bad


# ---- random structure: quoted data with comments, strings, odd tokens, every kind of whitespace ----------
def _rand_datum(r: random.Random, d: int) -> str:
    k = r.random()
    if d <= 0 or k < 0.45:
        return r.choice([
            str(r.randint(-10 ** 6, 10 ** 6)), repr(r.uniform(-1e3, 1e3)), "nil", "T", "()",
            r.choice(["a", "foo", "x1", "1+", "+", "-", "...", "a'b", 'q"r', "a;b", "E", "e5", ".", "1e",
                      "|||", "quote", "if", "lambda", "sym-%d" % r.randint(0, 50)]),
            '"%s"' % r.choice(["", "hi there", "a (b) c", "semi ; colon", "it's", " tab\t"]),
        ])
    if k < 0.55:
        return "'" + _rand_datum(r, d - 1)
    n = r.randint(0, 5)
    seps = [" ", "  ", "\t", "\n", " ; comment ( \" '\n", "\r\n", "\f", "\v"]
    inner = "".join(r.choice(seps) + _rand_datum(r, d - 1) for _ in range(n))
    return "(" + inner.lstrip(" ") + r.choice(["", " ", "\n"]) + ")"


def test_random_quoted_structure(culi, oracle_mod):
    r = random.Random(11)
    forms = []
    for _ in range(3000):
        d = _rand_datum(r, r.randint(0, 6))
        forms.append("'" + d if r.random() < 0.5 else "(quote %s)" % d)
    text = "\n".join(forms)
    assert len(text) > 3 * 4096                          # many lexer tiles, constructs across tile edges
    text_parity(culi, oracle_mod, "", text)


def test_long_tokens_strings_comments_across_tiles(culi, oracle_mod):
    long_sym = "s" * 9000
    long_str = '"' + ("x (y) ; z " * 1200) + '"'
    forms = "\n".join([
        "; " + "c" * 10000,
        "(quote %s)" % long_sym,
        "(list %s 1 2)" % long_str,
        "'(%s)" % " ".join(str(i) for i in range(5000)),
        "(length '(%s))" % " ".join("(a . b)" if False else "(a b)" for _ in range(3000)),
        '"' + "q" * 5000 + '"',
    ])
    text_parity(culi, oracle_mod, "", forms)


def test_symbols_shared_with_host_reader(culi, oracle_mod):
    """Symbols first seen by the device reader get the host table's dense ids, and vice versa."""
    ctx = culi.Context(**SMALL)
    ctx.define_text("(define dev-only (lambda (x) (* x 3)))\n(define pair '(dev-sym host-sym))")
    ctx.define("(define host-only (lambda (x) (+ (dev-only x) 1)))")
    r1 = ctx.eval_batch("(host-only 4)\n(dev-only 5)\n(car pair)\n'fresh-host")
    r2 = ctx.eval_text("(host-only 4)\n(dev-only 5)\n(car (cdr pair))\n'fresh-host\n'fresh-dev")
    r3 = ctx.eval_batch("'fresh-dev\n(eq 'fresh-dev (quote fresh-dev))")
    assert r1.printed() == ["13", "15", "dev-sym", "fresh-host"]
    assert r2.printed() == ["13", "15", "host-sym", "fresh-host", "fresh-dev"]
    assert r3.printed() == ["fresh-dev", "T"]


def test_device_text_and_unaligned_pointer(culi, oracle_mod):
    import torch
    wl = W.c5(3000)
    ctx = culi.Context(**SMALL)
    ctx.define_text(wl.defs)
    raw = torch.frombuffer(bytearray(b"#" + wl.forms.encode()), dtype=torch.uint8).cuda()
    a = ctx.eval_text(raw[1:])                           # device pointer, 1 byte off alignment
    b = ctx.eval_text(raw[1:].cpu().pin_memory())        # page-locked host memory
    s = oracle_mod.Session()
    s.define(wl.defs)
    o = s.eval(wl.forms)
    for res in (a, b):
        bad = compare(res.printed(), res.steps(), o)
        assert not bad, bad


def test_upload_text_then_eval_uploaded(culi, oracle_mod):
    wl = W.c2(500, lo=0, hi=14)
    ctx = culi.Context(**SMALL)
    ctx.define(wl.defs)
    h, nf = ctx.upload_text(wl.forms)
    assert nf == 500
    for _ in range(3):
        ctx.eval_uploaded(h)
    res = ctx.fetch_results(h)
    ctx.release(h)
    s = oracle_mod.Session()
    s.define(wl.defs)
    bad = compare(res.printed(), res.steps(), s.eval(wl.forms))
    assert not bad, bad


def test_empty_and_comment_only(culi):
    ctx = culi.Context(**SMALL)
    assert len(ctx.eval_text("")) == 0
    assert len(ctx.eval_text("  ; nothing here\n\t\n")) == 0
    ctx.define_text("")


# ---- read errors: same offsets as the host reader (and the oracle) ----------------------------------
ERRORS = ["(+ 1 2", ")", "(a))", "(a) )", "(a ')", '"abc', '(a "b', "99999999999999999999",
          "(x 9223372036854775808)", "(x -9223372036854775809)", "'(a b", "(a) (b", "((a)", "a ; (\n (b",
          "(a \"x)\" (b)", "(1 2)\n(3 4))\n(5", "(p '\n)", "( ( ( (", "(\"unterminated ( ) ;", "1 2 ) 3",
          "(a (b\n;)\n", "('a 'b ') c"]


def test_error_offsets(culi, oracle_mod):
    ctx = culi.Context(**SMALL)
    s = oracle_mod.Session()
    for t in ERRORS:
        with pytest.raises(culi.ParseError) as eh:
            ctx.read(t)
        with pytest.raises(culi.ParseError) as ed:
            ctx.eval_text(t)
        assert ed.value.offset == eh.value.offset, (t, ed.value.offset, eh.value.offset)
        with pytest.raises(oracle_mod.OracleError) as eo:
            s.eval(t)
        assert str(eo.value).endswith("offset %d" % eh.value.offset), (t, str(eo.value), eh.value.offset)
    # a ' with no datum before the end: host and device readers report the quote (R6)
    for t in ["(a '", "'", "x '  ; c"]:
        with pytest.raises(culi.ParseError) as eh:
            ctx.read(t)
        with pytest.raises(culi.ParseError) as ed:
            ctx.eval_text(t)
        assert ed.value.offset == eh.value.offset == t.rindex("'"), t
    # the context stays usable after read errors
    assert ctx.eval_text("(+ 1 2)").printed() == ["3"]


# ---- numbers --------------------------------------------------------------------------------------------
def _bits(x: float) -> int:
    return struct.unpack("<Q", struct.pack("<d", x))[0]


def _exact_decimal(fr: Fraction) -> str:
    """Exact decimal text of a dyadic rational (finite expansion)."""
    num, den = fr.numerator, fr.denominator
    k = den.bit_length() - 1
    assert den == 1 << k
    digits = num * 5 ** k                                # num / 2^k = num * 5^k / 10^k
    return "%de-%d" % (digits, k) if k else "%d.0" % digits


def float_cases(seed: int = 7) -> list[str]:
    r = random.Random(seed)
    out = ["0.0", "-0.0", "0e0", "1.0", "-1.5", ".5", "5.", "-.5e-3", "+1.25E+2", "000123.4500e+002",
           "1e308", "1.7976931348623157e308", "1.7976931348623158e308", "1.7976931348623159e308", "1e309",
           "2.2250738585072014e-308", "2.2250738585072011e-308", "4.9406564584124654e-324", "5e-324",
           "2.4703282292062327e-324", "2.4703282292062328e-324", "1e-400", "9007199254740993.0",
           "9007199254740992.9999999999999999999", "0.1", "0.30000000000000004", "123456789012345678901234567890.0",
           "1" + "0" * 400 + ".0e-400", "0." + "0" * 350 + "1e350", "1e22", "1e23", "8.98846567431158e307",
           "4.35e-321", "1.000000000000000000000000000001", "3.14159265358979323846264338327950288419716939937510"]
    for _ in range(2000):                                # repr of random finite doubles (any exponent)
        x = struct.unpack("<d", struct.pack("<Q", r.getrandbits(64)))[0]
        if x == x and abs(x) != float("inf"):
            out.append(repr(x) if "e" in repr(x) or "." in repr(x) else repr(x) + ".0")
    for _ in range(2000):                                # uniform(-4, 4) as in C3
        out.append(repr(r.uniform(-4, 4)))
    for _ in range(1500):                                # 15..40 significant digits, random exponents
        nd = r.randint(15, 40)
        digs = str(r.randint(10 ** (nd - 1), 10 ** nd - 1))
        out.append("%s.%se%d" % (digs[0], digs[1:], r.randint(-330, 310)))
    for _ in range(600):                                 # exact midpoints between neighbours, and +/- a hair
        x = abs(struct.unpack("<d", struct.pack("<Q", r.getrandbits(63)))[0])
        if not (x == x) or x == float("inf") or x >= 1.7e308:
            continue
        import math
        y = math.nextafter(x, float("inf"))
        mid = (Fraction(x) + Fraction(y)) / 2
        s = _exact_decimal(mid)
        out.append(s)
        mant, ex = s.split("e-") if "e-" in s else (s[:-2], "0")
        out.append("%s00001e-%d" % (mant, int(ex) + 5))            # just above the midpoint
        out.append("%de-%d" % (int(mant) * 100000 - 1, int(ex) + 5))  # just below
        if r.random() < 0.1:
            out.append("%s%s1e-%d" % (mant, "0" * 800, int(ex) + 801))  # sticky digit beyond 780
    return out


def test_float_literals_bit_exact(culi):
    cases = float_cases()
    ctx = culi.Context(**SMALL)
    res = ctx.eval_text("\n".join(cases))
    assert len(res) == len(cases)
    bad = []
    for i, s in enumerate(cases):
        exp = float(s)                                   # Python: correctly rounded (round half even)
        t, e, st = res.info(i)
        got = res.float_value(i)
        if _bits(got) != _bits(exp) or st != 1:
            bad.append((s[:60], got, exp))
    assert not bad, bad[:10]
    # and the host reader / oracle agree on the same text
    host = ctx.eval_batch("\n".join(cases))
    assert all(_bits(host.float_value(i)) == _bits(res.float_value(i)) for i in range(len(cases)))


def test_int_literals(culi):
    r = random.Random(3)
    cases = ["0", "-0", "+0", "0007", "9223372036854775807", "-9223372036854775808", "+9223372036854775807",
             "-" + "0" * 40 + "5"] + [str(r.randint(-2 ** 63, 2 ** 63 - 1)) for _ in range(3000)]
    ctx = culi.Context(**SMALL)
    res = ctx.eval_text("\n".join(cases))
    assert [res.int_value(i) for i in range(len(cases))] == [int(c) for c in cases]


def test_small_host_text_uses_host_reader(culi, oracle_mod):
    """Without CULI_F_DEVICE_READ, culi_eval_text reads host text of <= 16 KiB with the host reader (faster than
    the device reader's launches at that size): the same results and steps as the device
    reader and the oracle, wide lists (length marks) included; larger texts still go to the device."""
    import os as _os
    forms = "\n".join(["(fib 12)", "(fact 10)", "(sum 30)", "(||| 3 + '(1 2 3) '(4 5 6))", '"str"', "'(a b)",
                        "(||| 100 fib (%s))" % " ".join(["7"] * 100), "(length (list %s))" % " ".join(["1"] * 90)])
    old = _os.environ.get("CULI_DEVICE_READ")
    _os.environ["CULI_DEVICE_READ"] = "0"
    try:
        ctx = culi.Context(**SMALL)
    finally:
        _os.environ["CULI_DEVICE_READ"] = old if old is not None else "1"
    ctx.define(DEFS)
    r_host = ctx.eval_text(forms)
    ctx.last_stats()
    assert ctx.last_nested == 2                      # both wide lists suspended (host length marks)
    ctx_dev = culi.Context(**SMALL, flags=culi.CULI_F_DEVICE_READ)
    ctx_dev.define(DEFS)
    r_dev = ctx_dev.eval_text(forms)
    assert (r_host.printed(), r_host.steps()) == (r_dev.printed(), r_dev.steps())
    o = oracle_mod.Session()
    o.define(DEFS)
    exp = o.eval_batch(forms, nthreads=1).results
    assert not compare(r_host.printed(), r_host.steps(), exp, forms.splitlines())
