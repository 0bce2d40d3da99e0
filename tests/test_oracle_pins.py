"""Pins for the oracle (oracle/culi_oracle.cpp) against things other than itself:
the paper's worked examples, closed forms, brute force on tiny inputs with Python's own integers,
floats and lists, and invariants.  None of these retype the oracle's code: every expected value here
is computed by Python semantics (big integers reduced mod 2**64, IEEE floats, lists) or printed in the
paper / SURVEY §8(c).12b.
"""
from __future__ import annotations

import itertools
import math
import os
import random

import pytest

from paper_conf_cluster_subdbn18_b200 import workloads as W

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")


def load_tsv(name):
    rows = []
    with open(os.path.join(GOLDEN, name)) as f:
        for line in f:
            if not line.strip() or line.startswith("#"):
                continue
            parts = line.rstrip("\n").split("\t")
            rows.append(parts)
    return rows


@pytest.fixture()
def sess(oracle_mod):
    s = oracle_mod.Session()
    s.define("\n".join([W.FIB_DEF, W.FACT_DEF, W.SUM_DEF, W.WHEN_DEF]))
    return s


def wrap64(v: int) -> int:
    return (v + 2**63) % 2**64 - 2**63


def fib_py(n: int) -> int:
    a, b = 0, 1
    for _ in range(n):
        a, b = b, a + b
    return a


# ---- paper worked examples (tests/golden/paper_examples.tsv, each row cites PAPER.md) ---------------
@pytest.mark.parametrize("row", load_tsv("paper_examples.tsv"), ids=lambda r: r[0][:40])
def test_paper_examples(sess, row):
    form, expected, steps = row[0], row[1], int(row[2])
    r = sess.eval1(form)
    assert r.printed == expected
    assert r.steps == steps


# ---- SURVEY §8(c).12b step/semantics pins ---------------------------------------------------------
@pytest.mark.parametrize("row", load_tsv("step_pins.tsv"), ids=lambda r: r[0][:40])
def test_step_pins(sess, row):
    form, expected, steps = row[0], row[1], int(row[2])
    r = sess.eval1(form)
    assert (r.printed, r.steps) == (expected, steps)


# ---- closed forms (c.12) -------------------------------------------------------------------------
def test_fib_closed_form(sess):
    ns = list(range(0, 23))
    res = sess.eval("\n".join("(fib %d)" % n for n in ns))
    for n, r in zip(ns, res):
        assert r.err == 0
        assert int(r.printed) == fib_py(n)
        # S_fib(n) = 27 F(n+1) - 17, from the recurrence body(n) = 20 + body(n-1) + body(n-2)
        assert r.steps == 27 * fib_py(n + 1) - 17


def test_fact_closed_form(sess):
    ns = list(range(0, 26))
    res = sess.eval("\n".join("(fact %d)" % n for n in ns))
    for n, r in zip(ns, res):
        assert int(r.printed) == wrap64(math.factorial(n))     # int64 two's-complement wrap
        assert r.steps == (15 * n - 5 if n >= 2 else 10)


def test_sum_closed_form_and_depth_limit(sess):
    ns = [0, 1, 2, 10, 100, 300, 340]
    res = sess.eval("\n".join("(sum %d)" % n for n in ns))
    for n, r in zip(ns, res):
        assert int(r.printed) == n * (n + 1) // 2
        assert r.steps == 15 * n + 10
    # depth grows by 3 per recursion level: (sum n) needs depth 3n+4 -> 341 is the first failure at 1024
    assert sess.eval1("(sum 340)").printed == str(340 * 341 // 2)
    r = sess.eval1("(sum 341)")
    assert r.printed == "#<error DEPTH>"
    assert sess.eval1("(sum 400)").printed == "#<error DEPTH>"


def test_depth_limit_is_exact(oracle_mod):
    # (sum n) reaches depth 3n+4; with max_depth = 3n+4 it succeeds, with 3n+3 it fails.
    for n in (5, 17, 40):
        ok = oracle_mod.Session(max_depth=3 * n + 4)
        ok.define(W.SUM_DEF)
        assert ok.eval1("(sum %d)" % n).printed == str(n * (n + 1) // 2)
        bad = oracle_mod.Session(max_depth=3 * n + 3)
        bad.define(W.SUM_DEF)
        assert bad.eval1("(sum %d)" % n).printed == "#<error DEPTH>"


def test_fuel_limit(oracle_mod):
    s = oracle_mod.Session(fuel=198)
    s.define(W.FIB_DEF)
    r = s.eval1("(fib 5)")                 # needs 199 steps
    assert (r.printed, r.steps) == ("#<error FUEL>", 199)
    s2 = oracle_mod.Session(fuel=199)
    s2.define(W.FIB_DEF)
    assert s2.eval1("(fib 5)").printed == "5"


def test_int64_wrap_random(sess):
    rnd = random.Random(11)
    forms, exp = [], []
    for _ in range(500):
        a, b, c = (rnd.randrange(-2**63, 2**63) for _ in range(3))
        op1, op2 = rnd.choice("+-*"), rnd.choice("+-*")
        f = lambda o, x, y: {"+": x + y, "-": x - y, "*": x * y}[o]
        forms.append("(%s (%s %d %d) %d)" % (op2, op1, a, b, c))
        exp.append(wrap64(f(op2, wrap64(f(op1, a, b)), c)))
    res = sess.eval("\n".join(forms))
    assert [int(r.printed) for r in res] == exp


def _trunc_div(a, b):
    q = abs(a) // abs(b)
    return q if (a >= 0) == (b > 0) else -q


def test_division_rem_mod_bruteforce(sess):
    vals = list(range(-7, 8)) + [2**63 - 1, -2**63, 2**62 + 3, -(2**62) - 5]
    forms, exp = [], []
    for a in vals:
        for b in vals:
            for op in ("/", "rem", "mod"):
                forms.append("(%s %d %d)" % (op, a, b))
                if b == 0:
                    exp.append("#<error DIV0>")
                elif op == "/":
                    exp.append(str(wrap64(_trunc_div(a, b))))
                elif op == "rem":
                    exp.append(str(a - b * _trunc_div(a, b)))
                else:
                    exp.append(str(a % b))            # Python % is floor mod (sign of the divisor)
    res = sess.eval("\n".join(forms))
    assert [r.printed for r in res] == exp


def test_float_arith_bit_exact(sess):
    rnd = random.Random(3)
    forms, exp = [], []
    for _ in range(400):
        a, b, c = (rnd.uniform(-1e3, 1e3) for _ in range(3))
        forms.append("(/ (+ (* %r %r) %r) 2.0)" % (a, b, c))
        exp.append((a * b + c) / 2.0)
        forms.append("(- %r %r %r)" % (a, b, c))
        exp.append(a - b - c)
        forms.append("(sqrt %r)" % abs(a))
        exp.append(math.sqrt(abs(a)))
    res = sess.eval("\n".join(forms))
    for r, e in zip(res, exp):
        assert float(r.printed) == e                # bit-exact (shortest repr round-trips)


def test_mixed_int_float_fold(sess):
    # left fold from the first argument; an INT accumulator switches to f64 at the first FLOAT step
    r = sess.eval("(+ 9007199254740993 1 0.5)\n(+ 9007199254740993 0.5 1)\n(* 3 0.5 3)\n(- 5)\n(- 2.5)")
    assert float(r[0].printed) == float(9007199254740994) + 0.5
    assert float(r[1].printed) == (float(9007199254740993) + 0.5) + 1.0
    assert r[2].printed == "4.5"
    assert r[3].printed == "-5"
    assert r[4].printed == "-2.5"


def test_c3_closure_float(oracle_mod):
    wl = W.c3(64)
    s = oracle_mod.Session()
    s.define(wl.defs)
    xs = [float(t) for t in wl.defs.split("'(")[1].rstrip(")\n").split()]
    r = s.eval1(wl.forms)
    got = [float(t) for t in r.printed.strip("()").split()]
    exp = [((0.75 * x) * (0.75 * x) + (x + 1.5)) / 2.0 for x in xs]
    assert got == exp
    assert r.steps == 5 + 20 * 64


# ---- brute force: list builtins against Python lists -----------------------------------------------
def _lisp(xs):
    if xs is None:
        return "nil"
    return "(" + " ".join(str(x) for x in xs) + ")" if xs else "nil"


def test_list_builtins_bruteforce(sess):
    rnd = random.Random(5)
    forms, exp = [], []
    for _ in range(300):
        a = [rnd.randint(-9, 9) for _ in range(rnd.randint(0, 5))]
        b = [rnd.randint(-9, 9) for _ in range(rnd.randint(0, 5))]
        la, lb = "(list%s)" % "".join(" %d" % v for v in a), "(list%s)" % "".join(" %d" % v for v in b)
        k = rnd.randint(0, 6)
        forms += ["(append %s %s)" % (la, lb), "(reverse %s)" % la, "(length %s)" % la,
                  "(nth %d %s)" % (k, la), "(car %s)" % la, "(cdr %s)" % la,
                  "(cons %d %s)" % (k, lb), "(equal %s %s)" % (la, lb),
                  "(append %s)" % la, "(append %s %s %s)" % (la, lb, la)]
        exp += [_lisp(a + b), _lisp(a[::-1]), str(len(a)),
                str(a[k]) if k < len(a) else "nil", str(a[0]) if a else "nil", _lisp(a[1:]),
                _lisp([k] + b), "T" if a == b else "nil", _lisp(a), _lisp(a + b + a)]
    res = sess.eval("\n".join(forms))
    assert [r.printed for r in res] == exp


def test_list_errors_and_edges(sess):
    cases = {r[0]: r[1] for r in load_tsv("edge_cases.tsv")}
    forms = list(cases)
    res = sess.eval("\n".join(forms))
    got = {f: r.printed for f, r in zip(forms, res)}
    assert got == cases


def test_dotted_data_is_a_symbol_not_syntax(sess):
    # c.1 has no dotted-pair syntax: "." reads as a symbol; improper lists only come from cons
    r = sess.eval1("(list 1 . 2)")
    assert r.printed == "(1 . 2)"
    r = sess.eval1("(car (list (cons 1 2)))")
    assert r.printed == "(1 . 2)"


def test_eval_of_improper_list_is_syntax_error(oracle_mod):
    s = oracle_mod.Session()
    s.define("(defmacro bad () (cons 1 2))")
    r = s.eval1("(bad)")
    assert r.printed == "#<error SYNTAX>"
    assert r.steps == 2 + 4 + 1                        # list + head, body (cons 1 2), then the expansion


# ---- invariants --------------------------------------------------------------------------------------
def test_macro_equals_hand_expansion(sess, oracle_mod):
    rnd = random.Random(9)
    for _ in range(100):
        c = rnd.choice(["(< %d %d)" % (rnd.randint(-3, 3), rnd.randint(-3, 3)), "nil", "T", "1"])
        x = "(+ %d %d)" % (rnd.randint(-9, 9), rnd.randint(-9, 9))
        m = sess.eval1("(when %s %s)" % (c, x))
        h = sess.eval1("(if %s %s nil)" % (c, x))
        assert m.printed == h.printed
        # expansion body (list 'if c x nil) costs 7 steps; the macro call adds list + head
        assert m.steps == 2 + 7 + h.steps


def test_par_equals_sequential_map(sess):
    rnd = random.Random(4)
    for _ in range(30):
        n = rnd.randint(0, 8)
        a = [rnd.randint(0, 12) for _ in range(n + rnd.randint(0, 2))]
        b = [rnd.randint(-5, 5) for _ in range(n + rnd.randint(0, 2))]
        la, lb = "(%s)" % " ".join(map(str, a)) if a else "nil", "(%s)" % " ".join(map(str, b)) if b else "nil"
        par = sess.eval1("(||| %d fib '%s)" % (n, la))
        seq = sess.eval1("(list%s)" % "".join(" (fib %d)" % v for v in a[:n]))
        assert par.printed == seq.printed
        par2 = sess.eval1("(||| %d - '%s '%s)" % (n, la, lb))
        assert par2.printed == _lisp([wrap64(x - y) for x, y in zip(a[:n], b[:n])])


def test_print_read_idempotent(sess, oracle_mod):
    rnd = random.Random(2)

    def datum(d):
        k = rnd.randint(0, 6 if d < 3 else 4)
        if k == 0:
            return str(rnd.randint(-10**18, 10**18))
        if k == 1:
            return repr(rnd.uniform(-1e6, 1e6))
        if k == 2:
            return rnd.choice(["a", "foo-bar", "|||", "+", "E", "1+", "x.y", "nil", "T"])
        if k == 3:
            return '"s %d"' % rnd.randint(0, 9)
        if k == 4:
            return repr(rnd.choice([1e300, -0.0, 5e-324, 1.5, 2.0, 1e16, 123456.789]))
        return "(%s)" % " ".join(datum(d + 1) for _ in range(rnd.randint(0, 4)))

    text = "\n".join(datum(0) for _ in range(300))
    once = sess.read_print(text)
    twice = sess.read_print("\n".join(once))
    assert once == twice


def test_reader_classification(sess):
    toks = {"+": "+", "-": "-", "E": "E", "1+": "1+", "+5": "5", "-0": "0", "1.": "1.0", ".5": "0.5",
            "1e3": "1000.0", "1E-2": "0.01", "-.5e1": "-5.0", "1.5.2": "1.5.2", "e5": "e5",
            "nil": "nil", "T": "T", "t": "t", "NIL": "NIL", "()": "nil", "|||": "|||"}
    out = sess.read_print("\n".join(toks))
    assert dict(zip(toks, out)) == toks


def test_reader_errors(oracle_mod):
    s = oracle_mod.Session()
    for bad in ["(+ 1 2", ")", "(a))", '"abc', "99999999999999999999", "'"]:
        with pytest.raises(oracle_mod.OracleError):
            s.read_print(bad)


def test_global_persistence(oracle_mod):
    # the environment persists across inputs; late binding (L447-448)
    s = oracle_mod.Session()
    s.define("(define k 1) (define g (lambda (x) (+ x k)))")
    assert s.eval1("(g 10)").printed == "11"
    s.define("(define k 5)")
    assert s.eval1("(g 10)").printed == "15"


def test_define_failure_leaves_no_binding(oracle_mod):
    s = oracle_mod.Session()
    with pytest.raises(oracle_mod.OracleError, match="form 1: DIV0"):
        s.define("(define a 1) (define b (/ 1 0)) (define c 3)")
    assert s.eval("a\nb\nc") and [r.printed for r in s.eval("a\nb\nc")] == ["1", "b", "c"]


def test_generators_deterministic():
    for name, gen, kw in [("C1", W.c1, {"n": 50}), ("C2", W.c2, {"n": 50}), ("C4", W.c4, {"n": 50}),
                          ("C5", W.c5, {"n": 50}), ("C3", W.c3, {"n": 50})]:
        a, b = gen(**kw), gen(**kw)
        assert a.sha256() == b.sha256(), name


def test_generated_batches_run_clean(oracle_mod):
    # every generated form evaluates without an error under the oracle (sanity of the recipes)
    for wl in (W.c1(200), W.c2(40, lo=5, hi=12), W.c4(300), W.c5(300)):
        s = oracle_mod.Session()
        if wl.defs:
            s.define(wl.defs)
        res = s.eval(wl.forms)
        assert len(res) == wl.nforms
        assert all(r.err == 0 for r in res), [r for r in res if r.err][:3]


SETQ_DEFS = "\n".join([
    "(define make-counter (lambda () (let ((n 0)) (lambda () (setq n (+ n 1))))))",
    "(define counter (let ((n 0)) (lambda () (setq n (+ n 1)))))",
    "(define g 7)",
    "(define k1 (counter))",
    "(define k2 (counter))",
])


@pytest.fixture(scope="module")
def setq_sess(oracle_mod):
    s = oracle_mod.Session()
    s.define(SETQ_DEFS)
    return s


@pytest.mark.parametrize("row", load_tsv("setq_pins.tsv"), ids=lambda r: r[0][:40])
def test_setq_pins(setq_sess, row):
    """setq under reading R7: hand-derived values and step counts."""
    r = setq_sess.eval1(row[0])
    assert (r.printed, r.steps) == (row[1], int(row[2])), row


def test_setq_define_time_globals(oracle_mod):
    """At define time setq updates (or creates) the global binding; batches see the result (L408-413)."""
    s = oracle_mod.Session()
    s.define("(define a 1)\n(setq a (+ a 41))\n(setq fresh 'made)\n(define f (lambda () a))")
    assert [r.printed for r in s.eval("a\nfresh\n(f)")] == ["42", "made", "42"]


def test_setq_counter_closed_form(oracle_mod):
    """A counter closure called k times in one form returns k; steps = 9 + 8k (let 2 + make-counter 7 + k calls)."""
    s = oracle_mod.Session()
    s.define(SETQ_DEFS)
    for k in (1, 2, 5, 17):
        r = s.eval1("(let ((c (make-counter))) %s)" % " ".join(["(c)"] * k))
        assert (r.printed, r.steps) == (str(k), 9 + 8 * k)


def test_setq_forms_are_independent(oracle_mod):
    """Two forms of one batch each get their own counter: no state leaks between independent forms."""
    s = oracle_mod.Session()
    s.define(SETQ_DEFS)
    out = [r.printed for r in s.eval("(let ((c (make-counter))) (c) (c))\n(let ((c (make-counter))) (c))")]
    assert out == ["2", "1"]


# ---- defun (§III-A.b: function forms "stored in the global environment by the
# keyword defun"; SURVEY c.5 / c.13 #12: defun is sugar for define + lambda, no extra steps) --------------
DEFUN_DEFS = "\n".join([
    "(defun sq (x) (* x x))",
    "(defun k42 () 42)",
    "(defun two (x) (+ x 1) (* x 2))",
    "(defun fibd (n) (if (< n 2) n (+ (fibd (- n 1)) (fibd (- n 2)))))",
    "(defun factd (n) (if (< n 2) 1 (* n (factd (- n 1)))))",
    "(defun add3 (a b c) (+ a (* 10 b) (* 100 c)))",
    "(defun firstp (a a) a)",
])


@pytest.fixture(scope="module")
def defun_sess(oracle_mod):
    s = oracle_mod.Session()
    s.define(DEFUN_DEFS)
    return s


def test_defun_hand_derived(defun_sess):
    # steps by c.4: (sq 7) = list 1 + head 1 + arg 1 + body (* x x) 4 = 7; (k42) = 2 + body atom 1 = 3;
    # (two 5) = 3 + (+ x 1) 4 + (* x 2) 4 = 11; (add3 1 2 3) = 5 + body: list+head 2, a 1, (* 10 b) 4,
    # (* 100 c) 4 = 16
    cases = [("(sq 7)", "49", 7), ("(k42)", "42", 3), ("(two 5)", "10", 11), ("(add3 1 2 3)", "321", 16),
             ("(firstp 1 2)", "1", 5), ("sq", "#<lambda>", 1), ("(sq)", "#<error ARITY>", 2),
             ("(sq 1 2)", "#<error ARITY>", 4), ("(k42 1)", "#<error ARITY>", 3),
             ("(sq 'a)", "#<error TYPE>", 8)]
    res = defun_sess.eval("\n".join(c[0] for c in cases))
    assert [(r.printed, r.steps) for r in res] == [(c[1], c[2]) for c in cases]


def test_defun_closed_forms(defun_sess):
    # the recurrences of c.12 hold unchanged for the defun-defined functions (defun adds no steps)
    ns = list(range(0, 21))
    res = defun_sess.eval("\n".join("(fibd %d)" % n for n in ns))
    for n, r in zip(ns, res):
        assert (int(r.printed), r.steps) == (fib_py(n), 27 * fib_py(n + 1) - 17)
    res = defun_sess.eval("\n".join("(factd %d)" % n for n in ns))
    for n, r in zip(ns, res):
        assert (int(r.printed), r.steps) == (wrap64(math.factorial(n)), 15 * n - 5 if n >= 2 else 10)


def test_defun_equals_define_lambda(oracle_mod, defun_sess):
    # c.13 #12: defun is sugar — same value and same step count as the define + lambda spelling
    s = oracle_mod.Session()
    s.define("\n".join([
        "(define sq (lambda (x) (* x x)))", "(define two (lambda (x) (+ x 1) (* x 2)))",
        "(define fibd (lambda (n) (if (< n 2) n (+ (fibd (- n 1)) (fibd (- n 2))))))"]))
    forms = "\n".join(["(sq 12)", "(two -3)", "(fibd 12)", "(list (sq 3) (two 4))", "(||| 3 sq '(1 2 3))"])
    a = [(r.printed, r.steps) for r in s.eval(forms)]
    b = [(r.printed, r.steps) for r in defun_sess.eval(forms)]
    assert a == b


def test_defun_syntax_errors(oracle_mod):
    # reserved name, non-list parameters, reserved parameter, missing body: SYNTAX (c.5), no binding made
    for bad in ["(defun if (x) x)", "(defun f x x)", "(defun f (car) car)", "(defun f)", "(defun 5 (x) x)"]:
        s = oracle_mod.Session()
        with pytest.raises(oracle_mod.OracleError, match="SYNTAX"):
            s.define(bad)
    s = oracle_mod.Session()
    s.define("(defun f () )")                               # empty body -> nil (c.4)
    assert (s.eval1("(f)").printed, s.eval1("(f)").steps) == ("nil", 2)


def test_defun_redefinition_late_binding(oracle_mod):
    # PAPER L98-101 / L447-448: a redefinition via defun is seen by existing callers
    s = oracle_mod.Session()
    s.define("(defun g (x) (+ x 1))\n(defun h (x) (g (g x)))")
    assert s.eval1("(h 1)").printed == "3"
    s.define("(defun g (x) (* x 10))")
    assert s.eval1("(h 1)").printed == "100"


# ---- comparisons (c.6: numeric, mixed -> f64, IEEE: nan compares false) against Python --------------------
_CMP_INTS = [-2, -1, 0, 1, 2, 9007199254740992, 9007199254740993, -2**63, 2**63 - 1]
_CMP_FLOATS = ["-1.5", "-0.0", "0.0", "0.5", "1.0", "2.0", "9007199254740992.0", "1e300", "-1e300"]
_CMP_SPECIAL = {"(/ 1 0.0)": math.inf, "(/ -1 0.0)": -math.inf, "(/ 0 0.0)": math.nan}


def _cmp_py(op, a, b):
    if isinstance(a, float) or isinstance(b, float):
        a, b = float(a), float(b)                             # Python int -> float rounds to nearest even
    return {"=": a == b, "<": a < b, ">": a > b, "<=": a <= b, ">=": a >= b}[op]


def test_comparisons_bruteforce(sess):
    vals = [(str(v), v) for v in _CMP_INTS] + [(t, float(t)) for t in _CMP_FLOATS] + list(_CMP_SPECIAL.items())
    forms, exp = [], []
    for op in ("=", "<", ">", "<=", ">="):
        for (ta, va), (tb, vb) in itertools.product(vals, vals):
            forms.append("(%s %s %s)" % (op, ta, tb))
            exp.append("T" if _cmp_py(op, va, vb) else "nil")
    res = sess.eval("\n".join(forms))
    got = [r.printed for r in res]
    bad = [(f, g, e) for f, g, e in zip(forms, got, exp) if g != e]
    assert not bad, bad[:10]
    # steps: list + head + 2 atom args = 4 for atom operands
    assert all(r.steps == 4 for f, r in zip(forms, res) if "(/" not in f)


def test_comparison_errors(sess):
    cases = [("(< 1)", "#<error ARITY>"), ("(>= 1 2 3)", "#<error ARITY>"), ("(<=)", "#<error ARITY>"),
             ("(= 1 'a)", "#<error TYPE>"), ("(> nil 1)", "#<error TYPE>"), ("(< \"s\" 1)", "#<error TYPE>"),
             ("(<= (list 1) 2)", "#<error TYPE>")]
    assert [r.printed for r in sess.eval("\n".join(c[0] for c in cases))] == [c[1] for c in cases]


# ---- brute force, exhaustive: EVERY arithmetic tree of op-depth <= 2 (mixed depths included) --------------
def _trees_upto(depth):
    """All trees of op-depth <= depth over {+,-,*} and leaves -2..2: (text, python value, op count)."""
    leaves = [(str(v), v, 0) for v in range(-2, 3)]
    if depth == 0:
        return leaves
    subs = _trees_upto(depth - 1)
    out = list(subs)
    seen = {t for t, _, _ in subs}
    for op in "+-*":
        for (ta, va, oa), (tb, vb, ob) in itertools.product(subs, subs):
            text = "(%s %s %s)" % (op, ta, tb)
            if text in seen:
                continue
            seen.add(text)
            out.append((text, {"+": va + vb, "-": va - vb, "*": va * vb}[op], oa + ob + 1))
    return out


def test_bruteforce_arith_trees_exhaustive(sess):
    trees = _trees_upto(2)
    assert len(trees) == 5 + 75 + 3 * (80 * 80 - 25)        # leaves, depth-1, depth-2 (any child mix)
    res = sess.eval("\n".join(t for t, _, _ in trees))
    for (text, val, ops), r in zip(trees, res):
        assert (int(r.printed), r.steps) == (wrap64(val), 3 * ops + 1), text


# ---- quasiquote (reading R8) --------------------------------------------------
@pytest.mark.parametrize("row", load_tsv("quasiquote_pins.tsv"), ids=lambda r: r[0][:40])
def test_quasiquote_pins(oracle_mod, row):
    s = oracle_mod.Session()
    r = s.eval1(row[0])
    assert (r.printed, r.steps) == (row[1], int(row[2])), row


def test_quasiquote_macro(oracle_mod):
    """A macro written with a quasiquote template expands to the same code as its list-built twin: same
    value; steps differ only by the construction cost of the expansion (R8: the walk is free, each unquote
    one step for a parameter symbol, vs. list + head + one step per list argument)."""
    s = oracle_mod.Session()
    s.define("(defmacro my-if (c a b) `(if ,c ,a ,b))\n(defmacro my-if2 (c a b) (list 'if c a b))")
    r1 = s.eval1("(my-if (< 1 2) 'yes 'no)")
    assert (r1.printed, r1.steps) == ("yes", 15)        # 2 call + 5 template (2 + c a b) + 8 expansion
    r2 = s.eval1("(my-if2 (< 1 2) 'yes 'no)")
    assert (r2.printed, r2.steps) == ("yes", 17)        # 2 call + 7 (list 'if c a b), as c.12b's when, + 8


def _qq_equiv(t):
    """Python model of R8 for flat templates: items are ('lit', x) | ('uq', expr, value) | ('spl', expr, list)."""
    out, text, steps = [], [], 2
    for it in t:
        if it[0] == "lit":
            out.append(it[1]); text.append(str(it[1]))
        elif it[0] == "uq":
            out.append(it[2]); text.append(",(+ %d %d)" % it[1]); steps += 4
        else:
            out.extend(it[2]); text.append("(unquote-splicing (list%s))" % "".join(" %d" % v for v in it[2]))
            steps += 2 + len(it[2])
    return "`(" + " ".join(text) + ")", ("(" + " ".join(map(str, out)) + ")") if out else "nil", steps


def test_quasiquote_bruteforce(oracle_mod):
    """Random flat templates against a Python model of R8 (values and step counts)."""
    rnd = random.Random(8)
    s = oracle_mod.Session()
    cases = []
    for _ in range(300):
        t = []
        for _ in range(rnd.randint(0, 6)):
            k = rnd.randint(0, 2)
            if k == 0:
                t.append(("lit", rnd.randint(-9, 9)))
            elif k == 1:
                a, b = rnd.randint(-9, 9), rnd.randint(-9, 9)
                t.append(("uq", (a, b), a + b))
            else:
                t.append(("spl", None, [rnd.randint(-9, 9) for _ in range(rnd.randint(0, 3))]))
        cases.append(_qq_equiv(t))
    res = s.eval("\n".join(c[0] for c in cases))
    for (text, printed, steps), r in zip(cases, res):
        assert (r.printed, r.steps) == (printed, steps), text


def test_quasiquote_reader(oracle_mod):
    s = oracle_mod.Session()
    assert s.read_print("`(a ,b)\n'`x\n,,y\na`b\nc,d") == [
        "(quasiquote (a (unquote b)))", "(quote (quasiquote x))", "(unquote (unquote y))", "a`b", "c,d"]
    for bad in ["`", "(a ,)", ",", "`)"]:
        with pytest.raises(oracle_mod.OracleError):
            s.read_print(bad)


# ---- float printing (SURVEY c.8 "shortest round trip"; reading R3) against Python's repr --------
def _sig_digits(s: str) -> int:
    m = s.lower().lstrip("-").split("e")[0].replace(".", "").lstrip("0").rstrip("0")
    return max(len(m), 1)


def test_float_printing_shortest_round_trip(sess):
    """Every printed FLOAT reads back to the same double (bit-exact, Python float()) with as few significant
    digits as Python's repr — an independent shortest-round-trip printer (David Gay / Ryu lineage) — and always
    carries a '.' or an exponent (so it reads back as FLOAT, c.1); nan / ±inf print as nan / inf / -inf.
    (std::to_chars picks plain notation when it is no longer than scientific; an integral value of 2^53 or
    more then prints as its exact integer digits, which also round-trips.)"""
    import struct
    rnd = random.Random(11)
    xs = [0.0, -0.0, 1.0, -2.5, 0.1, 1e16, 1e-5, 5e-324, 2.2250738585072014e-308, 1.7976931348623157e308,
          123456789012345678.0, 9007199254740993.0, 0.30000000000000004, 1e22, 1e21, 1e-7]
    xs += [rnd.uniform(-1e6, 1e6) for _ in range(300)]
    xs += [struct.unpack("<d", struct.pack("<Q", rnd.getrandbits(64)))[0] for _ in range(600)]
    xs = [x for x in xs if math.isfinite(x)]
    forms = ["(* %r 1.0)" % x for x in xs]             # a computed float, not the literal's text
    res = sess.eval("\n".join(forms))
    for x, r in zip(xs, res):
        p = r.printed
        assert float(p) == x and (math.copysign(1, float(p)) == math.copysign(1, x)), (x, p)
        assert "." in p or "e" in p.lower(), p
        if "e" not in p.lower() and abs(x) >= 2.0 ** 53:
            assert p == "%d.0" % int(x), (x, p)
        else:
            assert _sig_digits(p) == _sig_digits(repr(x)), (x, p, repr(x))
    r = sess.eval("(/ 1.0 0.0)\n(/ -1.0 0.0)\n(- (/ 1.0 0.0) (/ 1.0 0.0))")
    assert [x.printed for x in r] == ["inf", "-inf", "nan"]
