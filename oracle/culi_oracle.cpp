// =====================================================================================================
// culi_oracle.cpp — THE ORACLE.  TEST INFRASTRUCTURE ONLY.
//
// A plain, slow, obviously-correct, *recursive* CPU interpreter of the CuLi Lisp subset described in
// "And Now for Something Completely Different: Running Lisp on GPUs" (Süß, Döring, Brinkmann, Nagel),
// /root/reference/PAPER.md (cited below as "PAPER Lnnn §x"), with every ambiguity resolved the way
// SURVEY.md §8(c) reads it (cited as "c.N"); DESIGN.md §3 lists those readings.
//
// Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference legs may load or
// execute this file.  It shares NO code with the CUDA path (paper_conf_cluster_subdbn18_b200/): its own
// reader, its own values, its own environments, its own printer.  The product path never calls it.
//
// Method, step by step (§III-B Fig.5): read (L414-437) -> eval (L438-462) -> print
// (L463-475).  The canonical "eval step" is one entry into eval() (c.4); depth is the nesting level of
// eval() calls with the top-level form at depth 1 (c.10).
//
// Pinning: tests/test_oracle_*.py check this interpreter against the paper's worked
// examples (L284-287, L327-344, L560-589, L703), closed forms (fib / fact / sum and their step counts),
// brute force over tiny arithmetic trees and list compositions (Python integers / Python lists), and
// invariants (print∘read idempotence, macro ≡ hand expansion, ||| ≡ sequential map).  Functions whose
// exact semantics the paper never shows (error codes, the ||| length rule, float printing, eq on fresh
// lists) are pinned only by SURVEY §8(c): "parity unpinned" in that narrow sense.
//
// Build: g++ -std=c++17 -O2 -ffp-contract=off -fPIC -shared -pthread (no FMA contraction, c.9).
// =====================================================================================================
#include <atomic>
#include <charconv>
#include <chrono>
#include <cmath>
#include <cerrno>
#include <cstdint>
#include <cstdlib>
#include <cstring>
#include <deque>
#include <stdexcept>
#include <string>
#include <thread>
#include <unordered_map>
#include <utility>
#include <vector>

namespace oracle {

// ---- values (c.2; §III-A.b) ---------------------------------------------------------
enum Tag : uint8_t { NIL, TRUE_, INT, FLOAT, STRING, SYMBOL, CONS, BUILTIN, SPECIAL, CLOSURE, MACRO };

// error codes (c.10)
enum Err : int { E_OK = 0, E_TYPE = 1, E_ARITY = 2, E_DIV0 = 3, E_SYNTAX = 4, E_ARG = 5, E_DEPTH = 6,
                 E_FUEL = 7, E_DEFINE_IN_BATCH = 8, E_OOM = 9 };
static const char* kErrName[] = {"OK", "TYPE", "ARITY", "DIV0", "SYNTAX", "ARG", "DEPTH", "FUEL",
                                 "DEFINE_IN_BATCH", "OOM"};

struct Cell;
struct Closure;
struct Frame;

struct Val {
  Tag tag = NIL;
  union {
    int64_t i;
    double f;
    uint32_t sym;
    Cell* cell;
    Closure* clo;
    const std::string* str;
    int op;
  };
  Val() : i(0) {}
};

struct Cell { Val car, cdr; };                       // PAPER L326-333 Fig.2 (a cons cell)
struct Closure { Val params; Val body; const Frame* env; };   // c.5 lambda / defmacro (lexical env)
struct Frame {                                       // PAPER L383-398 §III-B.a Fig.6-7: (symbol,value)
  const Frame* parent;                               // pairs plus a parent link; only setq changes a
  std::vector<std::pair<uint32_t, Val>> binds;       // value (L408-413, R7)
  bool persistent;                                   // created while defining (culi_define)
};

struct LispError { int code; };

// ---- arena: everything a form allocates; dropped after the form is printed (c.13 #23) -------------
struct Arena {
  std::deque<Cell> cells;
  std::deque<Closure> closures;
  std::deque<Frame> frames;
  std::deque<std::string> strings;
  void reset() { cells.clear(); closures.clear(); frames.clear(); strings.clear(); }
};

// ---- reserved names: special forms (c.5) then builtins (c.6) -------------------------------------
enum Special { S_QUOTE, S_IF, S_DEFINE, S_DEFUN, S_DEFMACRO, S_LAMBDA, S_LET, S_PROGN, S_SETQ,
               S_QUASIQUOTE, S_UNQUOTE, S_UNQUOTE_SPLICING, N_SPECIAL };
static const char* kSpecialNames[N_SPECIAL] = {"quote", "if", "define", "defun", "defmacro",
                                               "lambda", "let", "progn", "setq",
                                               "quasiquote", "unquote", "unquote-splicing"};
enum Builtin {
  B_ADD, B_SUB, B_MUL, B_DIV, B_REM, B_MOD, B_SQRT, B_FLOAT, B_TRUNC,
  B_NUM_EQ, B_LT, B_GT, B_LE, B_GE, B_EQ, B_EQUAL, B_NULL, B_NOT,
  B_ATOM, B_CONSP, B_NUMBERP, B_SYMBOLP, B_CONS, B_CAR, B_CDR, B_LIST,
  B_LENGTH, B_APPEND, B_REVERSE, B_NTH, B_PAR, N_BUILTIN
};
static const char* kBuiltinNames[N_BUILTIN] = {
  "+", "-", "*", "/", "rem", "mod", "sqrt", "float", "trunc",
  "=", "<", ">", "<=", ">=", "eq", "equal", "null", "not",
  "atom", "consp", "numberp", "symbolp", "cons", "car", "cdr", "list",
  "length", "append", "reverse", "nth", "|||"};

// ---- session: symbol table + global environment (persists for the session) ---
struct Session {
  uint32_t max_depth;
  uint64_t fuel;
  std::unordered_map<std::string, uint32_t> symtab;
  std::vector<std::string> names;
  std::vector<Val> global_val;        // indexed by symbol id
  std::vector<char> global_bound;
  uint32_t n_reserved = 0;
  Arena persistent;                   // values created by define persist (L98-101)

  uint32_t intern(const std::string& s) {
    auto it = symtab.find(s);
    if (it != symtab.end()) return it->second;
    uint32_t id = (uint32_t)names.size();
    symtab.emplace(s, id);
    names.push_back(s);
    global_val.push_back(Val());
    global_bound.push_back(0);
    return id;
  }
  Session(uint32_t md, uint64_t fu) : max_depth(md), fuel(fu) {
    // The global environment holds the builtins.
    for (int k = 0; k < N_SPECIAL; ++k) {
      uint32_t id = intern(kSpecialNames[k]);
      Val v; v.tag = SPECIAL; v.op = k;
      global_val[id] = v; global_bound[id] = 1;
    }
    for (int k = 0; k < N_BUILTIN; ++k) {
      uint32_t id = intern(kBuiltinNames[k]);
      Val v; v.tag = BUILTIN; v.op = k;
      global_val[id] = v; global_bound[id] = 1;
    }
    n_reserved = (uint32_t)names.size();
  }
  bool reserved(uint32_t sym) const { return sym < n_reserved; }
};

// ---- helpers ---------------------------------------------------------------------------------------
static Val mk_int(int64_t i) { Val v; v.tag = INT; v.i = i; return v; }
static Val mk_float(double f) { Val v; v.tag = FLOAT; v.f = f; return v; }
static Val mk_sym(uint32_t s) { Val v; v.tag = SYMBOL; v.sym = s; return v; }
static Val mk_nil() { return Val(); }
static Val mk_t() { Val v; v.tag = TRUE_; return v; }
static Val mk_bool(bool b) { return b ? mk_t() : mk_nil(); }
static Val mk_cons(Arena& A, Val a, Val d) {
  A.cells.push_back(Cell{a, d});
  Val v; v.tag = CONS; v.cell = &A.cells.back(); return v;
}
static Val make_list(Arena& A, const std::vector<Val>& xs, Val tail) {
  Val r = tail;
  for (size_t k = xs.size(); k-- > 0;) r = mk_cons(A, xs[k], r);
  return r;
}
// A proper list ends in NIL (c.4 step 4).
static bool is_proper_list(Val x) {
  while (x.tag == CONS) x = x.cell->cdr;
  return x.tag == NIL;
}
static std::vector<Val> list_elems(Val x) {
  std::vector<Val> out;
  while (x.tag == CONS) { out.push_back(x.cell->car); x = x.cell->cdr; }
  return out;
}
[[noreturn]] static void fail(int code) { throw LispError{code}; }

// int64 arithmetic wraps (c.9, c.13 #16): computed in uint64_t and reinterpreted.
static int64_t wrap_add(int64_t a, int64_t b) { return (int64_t)((uint64_t)a + (uint64_t)b); }
static int64_t wrap_sub(int64_t a, int64_t b) { return (int64_t)((uint64_t)a - (uint64_t)b); }
static int64_t wrap_mul(int64_t a, int64_t b) { return (int64_t)((uint64_t)a * (uint64_t)b); }
static double as_f64(Val v) { return v.tag == INT ? (double)v.i : v.f; }   // INT->f64 is RN (c.9)
static bool is_num(Val v) { return v.tag == INT || v.tag == FLOAT; }

// ---- printer (§III-B.d; c.8) -----------------------------------------------------------
static void print_float(double d, std::string& out) {
  if (std::isnan(d)) { out += "nan"; return; }
  if (std::isinf(d)) { out += d < 0 ? "-inf" : "inf"; return; }
  char buf[64];
  auto r = std::to_chars(buf, buf + sizeof buf, d);    // shortest round-trip
  std::string s(buf, r.ptr);
  if (s.find_first_of(".e") == std::string::npos) s += ".0";
  out += s;
}
static void print_val(const Session& S, Val v, std::string& out) {
  switch (v.tag) {
    case NIL: out += "nil"; return;
    case TRUE_: out += "T"; return;
    case INT: out += std::to_string(v.i); return;
    case FLOAT: print_float(v.f, out); return;
    case STRING: out += '"'; out += *v.str; out += '"'; return;
    case SYMBOL: out += S.names[v.sym]; return;
    case BUILTIN: out += "#<builtin "; out += kBuiltinNames[v.op]; out += ">"; return;
    case SPECIAL: out += "#<special "; out += kSpecialNames[v.op]; out += ">"; return;
    case CLOSURE: out += "#<lambda>"; return;
    case MACRO: out += "#<macro>"; return;
    case CONS: {
      out += '(';
      Val x = v;
      bool first = true;
      while (x.tag == CONS) {
        if (!first) out += ' ';
        print_val(S, x.cell->car, out);
        first = false;
        x = x.cell->cdr;
      }
      if (x.tag != NIL) { out += " . "; print_val(S, x, out); }
      out += ')';
      return;
    }
  }
}

// ---- reader (§III-B.b; c.1) -----------------------------------------------------------
struct ReadError { size_t offset; };

static bool is_delim(char c) {
  return c == ' ' || c == '\t' || c == '\n' || c == '\r' || c == '\f' || c == '\v' || c == '(' ||
         c == ')';
}
static bool all_digits(const std::string& s, size_t a, size_t b) {
  if (a >= b) return false;
  for (size_t k = a; k < b; ++k) if (s[k] < '0' || s[k] > '9') return false;
  return true;
}
// ^[+-]?[0-9]+$
static bool looks_int(const std::string& t) {
  size_t a = (t[0] == '+' || t[0] == '-') ? 1 : 0;
  return all_digits(t, a, t.size());
}
// ^[+-]?([0-9]+\.[0-9]*|\.[0-9]+)([eE][+-]?[0-9]+)?$  or  ^[+-]?[0-9]+[eE][+-]?[0-9]+$
static bool looks_float(const std::string& t) {
  size_t k = (t[0] == '+' || t[0] == '-') ? 1 : 0;
  size_t e = t.find_first_of("eE", k);
  std::string mant = t.substr(k, (e == std::string::npos ? t.size() : e) - k);
  if (e != std::string::npos) {
    size_t x = e + 1;
    if (x < t.size() && (t[x] == '+' || t[x] == '-')) ++x;
    if (!all_digits(t, x, t.size())) return false;
  }
  size_t dot = mant.find('.');
  if (dot == std::string::npos) return e != std::string::npos && all_digits(mant, 0, mant.size());
  bool left = all_digits(mant, 0, dot), right = all_digits(mant, dot + 1, mant.size());
  bool right_empty = dot + 1 == mant.size();
  return (left && (right || right_empty)) || (dot == 0 && right);
}

struct Reader {
  Session& S;
  Arena& A;
  const std::string& src;
  size_t p = 0;
  Reader(Session& s, Arena& a, const std::string& t) : S(s), A(a), src(t) {}

  void skip_ws() {
    while (p < src.size()) {
      char c = src[p];
      if (c == ';') { while (p < src.size() && src[p] != '\n') ++p; continue; }
      if (c == ' ' || c == '\t' || c == '\n' || c == '\r' || c == '\f' || c == '\v') { ++p; continue; }
      break;
    }
  }
  bool at_end() { skip_ws(); return p >= src.size(); }

  Val atom(const std::string& t, size_t start) {
    if (t == "nil") return mk_nil();                    // L430-432
    if (t == "T") return mk_t();
    if (looks_int(t)) {
      errno = 0;
      char* end = nullptr;
      long long v = std::strtoll(t.c_str(), &end, 10);
      if (errno == ERANGE) throw ReadError{start};      // int64 out of range -> read error (c.1)
      return mk_int((int64_t)v);
    }
    if (looks_float(t)) return mk_float(std::strtod(t.c_str(), nullptr));   // RN (c.1)
    return mk_sym(S.intern(t));                         // everything else is a symbol (c.13 #2)
  }

  Val datum() {
    skip_ws();
    if (p >= src.size()) throw ReadError{p};
    char c = src[p];
    if (c == ')') throw ReadError{p};
    if (c == '\'' || c == '`' || c == ',') {            // 'x == (quote x); DESIGN R8: `x == (quasiquote x),
      ++p;                                              // ,x == (unquote x) (no ,@ shorthand)
      Val d = datum();
      const char* name = c == '\'' ? "quote" : c == '`' ? "quasiquote" : "unquote";
      return mk_cons(A, mk_sym(S.intern(name)), mk_cons(A, d, mk_nil()));
    }
    if (c == '(') {                                     // L416-421
      size_t open = p;
      ++p;
      std::vector<Val> items;
      for (;;) {
        skip_ws();
        if (p >= src.size()) throw ReadError{open};     // unbalanced (L484-486)
        if (src[p] == ')') { ++p; break; }
        items.push_back(datum());
      }
      return make_list(A, items, mk_nil());             // () -> nil
    }
    if (c == '"') {                                     // a string runs to the next '"' (c.13 #3)
      size_t q = src.find('"', p + 1);
      if (q == std::string::npos) throw ReadError{p};
      A.strings.push_back(src.substr(p + 1, q - p - 1));
      Val v; v.tag = STRING; v.str = &A.strings.back();
      p = q + 1;
      return v;
    }
    size_t start = p;
    while (p < src.size() && !is_delim(src[p])) ++p;
    return atom(src.substr(start, p - start), start);
  }

  std::vector<Val> all() {
    std::vector<Val> out;
    while (!at_end()) out.push_back(datum());
    return out;
  }
};

// ---- the interpreter (§III-B.c; c.4-c.7) -----------------------------------------------
struct Interp {
  Session& S;
  Arena& A;            // where this form's allocations go
  bool define_mode;    // culi_define (true) vs culi_eval_batch (false), c.5 / c.13 #25
  uint64_t steps = 0;

  Interp(Session& s, Arena& a, bool dm) : S(s), A(a), define_mode(dm) {}

  // lookup: innermost frame first, leftmost first inside a frame, then the global frame (L445-451)
  Val lookup(uint32_t sym, const Frame* env) {
    for (const Frame* f = env; f; f = f->parent)
      for (auto& b : f->binds)
        if (b.first == sym) return b.second;
    if (S.global_bound[sym]) return S.global_val[sym];
    return mk_sym(sym);                                 // an unbound symbol stays a symbol (L451)
  }

  bool bindable(Val s) { return s.tag == SYMBOL && !S.reserved(s.sym); }   // c.5 reserved names
  bool valid_params(Val ps) {
    if (!is_proper_list(ps)) return false;
    for (Val p : list_elems(ps)) if (!bindable(p)) return false;
    return true;
  }

  // c.4: one call = one canonical step
  Val eval(Val x, const Frame* env, uint32_t depth) {
    steps += 1;                                               // step 1
    if (steps > S.fuel) fail(E_FUEL);
    if (depth > S.max_depth) fail(E_DEPTH);
    switch (x.tag) {
      case SYMBOL: return lookup(x.sym, env);                 // step 3
      case CONS: break;
      default: return x;                                      // step 2 (L461-462)
    }
    if (!is_proper_list(x)) fail(E_SYNTAX);                   // step 4
    Val h = eval(x.cell->car, env, depth + 1);                // head always evaluated first (L440-441)
    Val rest = x.cell->cdr;
    switch (h.tag) {
      case SPECIAL: return apply_special(h.op, rest, env, depth);
      case BUILTIN: {
        std::vector<Val> args;
        for (Val a : list_elems(rest)) args.push_back(eval(a, env, depth + 1));
        return apply_builtin(h.op, args, depth);
      }
      case CLOSURE: {
        std::vector<Val> args;
        for (Val a : list_elems(rest)) args.push_back(eval(a, env, depth + 1));
        return apply_closure(h.clo, args, depth);
      }
      case MACRO: {                                          // c.4 MACRO branch, c.13 #13
        std::vector<Val> forms = list_elems(rest);
        std::vector<Val> ps = list_elems(h.clo->params);
        if (ps.size() != forms.size()) fail(E_ARITY);
        Frame* F = new_frame(h.clo->env);
        for (size_t k = 0; k < ps.size(); ++k) F->binds.emplace_back(ps[k].sym, forms[k]);
        Val expansion = mk_nil();
        for (Val b : list_elems(h.clo->body)) expansion = eval(b, F, depth + 1);
        return eval(expansion, env, depth + 1);              // expansion runs in the caller's env
      }
      default: {                                             // data list (L443-444, c.13 #8)
        std::vector<Val> vals{h};
        for (Val a : list_elems(rest)) vals.push_back(eval(a, env, depth + 1));
        return make_list(A, vals, mk_nil());
      }
    }
  }
  Frame* new_frame(const Frame* parent) {
    A.frames.push_back(Frame{parent, {}, define_mode});
    return &A.frames.back();
  }

  // closure application: new frame over the captured env, then the body as an implicit progn
  // (c.4 CLOSURE branch)
  Val apply_closure(const Closure* c, const std::vector<Val>& args, uint32_t depth) {
    std::vector<Val> ps = list_elems(c->params);
    if (ps.size() != args.size()) fail(E_ARITY);
    Frame* F = new_frame(c->env);
    for (size_t k = 0; k < ps.size(); ++k) F->binds.emplace_back(ps[k].sym, args[k]);
    Val r = mk_nil();
    for (Val b : list_elems(c->body)) r = eval(b, F, depth + 1);
    return r;
  }

  Val make_closure(Tag t, Val params, Val body, const Frame* env) {
    A.closures.push_back(Closure{params, body, env});
    Val v; v.tag = t; v.clo = &A.closures.back(); return v;
  }

  // ---- quasiquote (reading R8) ------------------------------------------------
  // qq(t, L): the template t at nesting level L.  An atom is itself (not evaluated).  (unquote e) at
  // level 1 is eval(e) at depth+1 of the quasiquote form; at a deeper level it is rebuilt as
  // (unquote qq(e, L-1)); (quasiquote e) inside is rebuilt as (quasiquote qq(e, L+1)).  Any other list is
  // rebuilt element by element, left to right; an element (unquote-splicing e) at level 1 evaluates e,
  // which must be a proper list (else TYPE), and its elements are copied in.  Every list of the template
  // is a fresh contiguous copy.  (unquote ...) / (unquote-splicing ...) / (quasiquote ...) with other than
  // one argument, (unquote-splicing e) not in an element position at level 1, and an improper template
  // list are SYNTAX errors, raised when the walk reaches them.  The walk itself takes no steps.
  bool is_op_list(Val t, int op) {
    return t.tag == CONS && t.cell->car.tag == SYMBOL && t.cell->car.sym == (uint32_t)op;
  }
  Val qq_arg(Val t) {                                   // the single argument of (op x), else SYNTAX
    if (!is_proper_list(t)) fail(E_SYNTAX);
    std::vector<Val> xs = list_elems(t);
    if (xs.size() != 2) fail(E_SYNTAX);
    return xs[1];
  }
  Val qq(Val t, int level, const Frame* env, uint32_t depth) {
    if (t.tag != CONS) return t;
    if (!is_proper_list(t)) fail(E_SYNTAX);
    if (is_op_list(t, S_UNQUOTE) && level == 1) return eval(qq_arg(t), env, depth + 1);
    if (is_op_list(t, S_UNQUOTE_SPLICING) && level == 1) fail(E_SYNTAX);   // not in an element position
    int rest_level = level;
    if (is_op_list(t, S_QUASIQUOTE)) { qq_arg(t); rest_level = level + 1; }
    else if (is_op_list(t, S_UNQUOTE) || is_op_list(t, S_UNQUOTE_SPLICING)) { qq_arg(t); rest_level = level - 1; }
    std::vector<Val> out;
    std::vector<Val> xs = list_elems(t);
    for (size_t k = 0; k < xs.size(); ++k) {
      int L = k == 0 ? level : rest_level;
      Val e = xs[k];
      if (L == 1 && is_op_list(e, S_UNQUOTE_SPLICING)) {
        Val v = eval(qq_arg(e), env, depth + 1);
        if (!is_proper_list(v)) fail(E_TYPE);
        for (Val y : list_elems(v)) out.push_back(y);
        continue;
      }
      out.push_back(qq(e, L, env, depth));
    }
    return make_list(A, out, mk_nil());
  }

  // ---- special forms (c.5): syntax checked before anything is evaluated; sub-evals at depth+1 ----
  Val apply_special(int op, Val rest, const Frame* env, uint32_t depth) {
    std::vector<Val> a = list_elems(rest);
    size_t n = a.size();
    switch (op) {
      case S_QUOTE:
        if (n != 1) fail(E_SYNTAX);
        return a[0];                                         // not evaluated, not copied
      case S_IF: {
        if (n != 2 && n != 3) fail(E_SYNTAX);
        Val c = eval(a[0], env, depth + 1);
        if (c.tag != NIL) return eval(a[1], env, depth + 1); // only NIL is false (L300-305)
        return n == 3 ? eval(a[2], env, depth + 1) : mk_nil();
      }
      case S_DEFINE: {
        if (!define_mode) fail(E_DEFINE_IN_BATCH);
        if (n != 2 || !bindable(a[0])) fail(E_SYNTAX);
        Val v = eval(a[1], env, depth + 1);
        S.global_val[a[0].sym] = v;                          // global frame (L316-319)
        S.global_bound[a[0].sym] = 1;
        return a[0];
      }
      case S_DEFUN:
      case S_DEFMACRO: {
        if (!define_mode) fail(E_DEFINE_IN_BATCH);
        if (n < 2 || !bindable(a[0]) || !valid_params(a[1])) fail(E_SYNTAX);
        Val body = rest.cell->cdr.cell->cdr;
        Val v = make_closure(op == S_DEFUN ? CLOSURE : MACRO, a[1], body, env);
        S.global_val[a[0].sym] = v;
        S.global_bound[a[0].sym] = 1;
        return a[0];
      }
      case S_LAMBDA:
        if (n < 1 || !valid_params(a[0])) fail(E_SYNTAX);
        return make_closure(CLOSURE, a[0], rest.cell->cdr, env);   // captures env (lexical, c.3)
      case S_LET: {                                          // c.13 #9: parallel let, new frame
        if (n < 1 || !is_proper_list(a[0])) fail(E_SYNTAX);
        std::vector<Val> bs = list_elems(a[0]);
        for (Val b : bs) {
          if (b.tag != CONS || !is_proper_list(b)) fail(E_SYNTAX);
          std::vector<Val> se = list_elems(b);
          if (se.size() != 2 || !bindable(se[0])) fail(E_SYNTAX);
        }
        std::vector<Val> vals;
        for (Val b : bs) vals.push_back(eval(list_elems(b)[1], env, depth + 1));   // outer env
        Frame* F = new_frame(env);
        for (size_t k = 0; k < bs.size(); ++k) F->binds.emplace_back(list_elems(bs[k])[0].sym, vals[k]);
        Val r = mk_nil();
        for (size_t k = 1; k < n; ++k) r = eval(a[k], F, depth + 1);
        return r;
      }
      case S_PROGN: {
        Val r = mk_nil();
        for (Val x : a) r = eval(x, env, depth + 1);
        return r;
      }
      case S_QUASIQUOTE:
        if (n != 1) fail(E_SYNTAX);
        return qq(a[0], 1, env, depth);
      case S_UNQUOTE:
      case S_UNQUOTE_SPLICING:
        fail(E_SYNTAX);                                      // only meaningful inside a quasiquote template
      case S_SETQ: {
        // "setq updates the nearest existing symbol that matches" — a local variable or,
        // failing that, the global one.  DESIGN.md R7: the value is evaluated first; during a batch the
        // global frame and frames made while defining are read-only (DEFINE_IN_BATCH), so independent
        // forms share no mutable state; with no binding anywhere, a define-time setq creates the global.
        if (n != 2 || !bindable(a[0])) fail(E_SYNTAX);
        Val v = eval(a[1], env, depth + 1);
        uint32_t sym = a[0].sym;
        for (const Frame* f = env; f; f = f->parent)
          for (auto& b : f->binds)
            if (b.first == sym) {
              if (!define_mode && f->persistent) fail(E_DEFINE_IN_BATCH);
              const_cast<std::pair<uint32_t, Val>&>(b).second = v;
              return v;
            }
        if (!define_mode) fail(E_DEFINE_IN_BATCH);
        S.global_val[sym] = v;
        S.global_bound[sym] = 1;
        return v;
      }
    }
    fail(E_SYNTAX);
  }

  // ---- builtins (c.6): args already evaluated; arity, then types left to right, then compute ------
  Val arith(int op, const std::vector<Val>& args) {
    size_t n = args.size();
    if ((op == B_SUB || op == B_DIV) && n == 0) fail(E_ARITY);
    for (Val v : args) if (!is_num(v)) fail(E_TYPE);
    if (n == 0) return mk_int(op == B_MUL ? 1 : 0);
    std::vector<Val> xs = args;
    if (n == 1 && op == B_SUB) {                             // unary minus
      if (xs[0].tag == INT) return mk_int(wrap_sub(0, xs[0].i));
      return mk_float(-xs[0].f);
    }
    if (n == 1 && op == B_DIV) xs.insert(xs.begin(), mk_int(1));   // (/ a) = (/ 1 a)
    Val acc = xs[0];                                        // left fold from the first argument (c.13 #29)
    for (size_t k = 1; k < xs.size(); ++k) {
      Val b = xs[k];
      if (acc.tag == INT && b.tag == INT) {
        switch (op) {
          case B_ADD: acc = mk_int(wrap_add(acc.i, b.i)); break;
          case B_SUB: acc = mk_int(wrap_sub(acc.i, b.i)); break;
          case B_MUL: acc = mk_int(wrap_mul(acc.i, b.i)); break;
          case B_DIV:
            if (b.i == 0) fail(E_DIV0);
            if (acc.i == INT64_MIN && b.i == -1) acc = mk_int(INT64_MIN);
            else acc = mk_int(acc.i / b.i);                 // truncates toward zero (c.13 #17)
            break;
        }
      } else {
        double x = as_f64(acc), y = as_f64(b);
        switch (op) {
          case B_ADD: acc = mk_float(x + y); break;
          case B_SUB: acc = mk_float(x - y); break;
          case B_MUL: acc = mk_float(x * y); break;
          case B_DIV: acc = mk_float(x / y); break;
        }
      }
    }
    return acc;
  }

  bool eq(Val a, Val b) {
    if (a.tag != b.tag) return false;
    switch (a.tag) {
      case NIL: case TRUE_: return true;
      case INT: return a.i == b.i;
      case FLOAT: { uint64_t x, y; std::memcpy(&x, &a.f, 8); std::memcpy(&y, &b.f, 8); return x == y; }
      case SYMBOL: return a.sym == b.sym;
      case CONS: return a.cell == b.cell;
      case STRING: return a.str == b.str;
      case CLOSURE: case MACRO: return a.clo == b.clo;
      case BUILTIN: case SPECIAL: return a.op == b.op;
    }
    return false;
  }
  bool equal(Val a, Val b) {
    while (a.tag == CONS && b.tag == CONS) {
      if (!equal(a.cell->car, b.cell->car)) return false;
      a = a.cell->cdr; b = b.cell->cdr;
    }
    if (a.tag == STRING && b.tag == STRING) return *a.str == *b.str;
    return eq(a, b);
  }

  Val apply_fn(Val f, const std::vector<Val>& args, uint32_t depth) {
    if (f.tag == BUILTIN) return apply_builtin(f.op, args, depth);
    return apply_closure(f.clo, args, depth);
  }

  Val apply_builtin(int op, const std::vector<Val>& a, uint32_t depth) {
    size_t n = a.size();
    auto need = [&](size_t k) { if (n != k) fail(E_ARITY); };
    switch (op) {
      case B_ADD: case B_SUB: case B_MUL: case B_DIV: return arith(op, a);
      case B_REM: case B_MOD: {
        need(2);
        if (a[0].tag != INT || a[1].tag != INT) fail(E_TYPE);
        int64_t x = a[0].i, y = a[1].i;
        if (y == 0) fail(E_DIV0);
        if (y == -1) return mk_int(0);                      // INT64_MIN rem -1 = 0
        int64_t r = x % y;                                  // C %: sign of the dividend
        if (op == B_MOD && r != 0 && ((r < 0) != (y < 0))) r += y;   // floor mod: sign of divisor
        return mk_int(r);
      }
      case B_SQRT:
        need(1);
        if (!is_num(a[0])) fail(E_TYPE);
        return mk_float(std::sqrt(as_f64(a[0])));
      case B_FLOAT:
        need(1);
        if (!is_num(a[0])) fail(E_TYPE);
        return mk_float(as_f64(a[0]));
      case B_TRUNC: {
        need(1);
        if (!is_num(a[0])) fail(E_TYPE);
        if (a[0].tag == INT) return a[0];
        double x = a[0].f;
        if (std::isnan(x) || std::fabs(x) >= 9223372036854775808.0) fail(E_ARG);
        return mk_int((int64_t)x);                          // toward zero
      }
      case B_NUM_EQ: case B_LT: case B_GT: case B_LE: case B_GE: {
        need(2);
        if (!is_num(a[0]) || !is_num(a[1])) fail(E_TYPE);
        if (a[0].tag == INT && a[1].tag == INT) {
          int64_t x = a[0].i, y = a[1].i;
          switch (op) {
            case B_NUM_EQ: return mk_bool(x == y);
            case B_LT: return mk_bool(x < y);
            case B_GT: return mk_bool(x > y);
            case B_LE: return mk_bool(x <= y);
            default: return mk_bool(x >= y);
          }
        }
        double x = as_f64(a[0]), y = as_f64(a[1]);
        switch (op) {
          case B_NUM_EQ: return mk_bool(x == y);
          case B_LT: return mk_bool(x < y);
          case B_GT: return mk_bool(x > y);
          case B_LE: return mk_bool(x <= y);
          default: return mk_bool(x >= y);
        }
      }
      case B_EQ: need(2); return mk_bool(eq(a[0], a[1]));
      case B_EQUAL: need(2); return mk_bool(equal(a[0], a[1]));
      case B_NULL: case B_NOT: need(1); return mk_bool(a[0].tag == NIL);
      case B_ATOM: need(1); return mk_bool(a[0].tag != CONS);
      case B_CONSP: need(1); return mk_bool(a[0].tag == CONS);
      case B_NUMBERP: need(1); return mk_bool(is_num(a[0]));
      case B_SYMBOLP: need(1); return mk_bool(a[0].tag == SYMBOL || a[0].tag == NIL || a[0].tag == TRUE_);
      case B_CONS: need(2); return mk_cons(A, a[0], a[1]);
      case B_CAR: case B_CDR:
        need(1);
        if (a[0].tag == NIL) return mk_nil();
        if (a[0].tag != CONS) fail(E_TYPE);
        return op == B_CAR ? a[0].cell->car : a[0].cell->cdr;
      case B_LIST: return make_list(A, a, mk_nil());
      case B_LENGTH:
        need(1);
        if (!is_proper_list(a[0])) fail(E_TYPE);
        return mk_int((int64_t)list_elems(a[0]).size());
      case B_APPEND: {
        if (n == 0) return mk_nil();
        for (size_t k = 0; k + 1 < n; ++k) if (!is_proper_list(a[k])) fail(E_TYPE);
        std::vector<Val> xs;
        for (size_t k = 0; k + 1 < n; ++k) for (Val e : list_elems(a[k])) xs.push_back(e);
        return make_list(A, xs, a[n - 1]);                   // shares the last argument
      }
      case B_REVERSE: {
        need(1);
        if (!is_proper_list(a[0])) fail(E_TYPE);
        std::vector<Val> xs = list_elems(a[0]);
        std::vector<Val> r(xs.rbegin(), xs.rend());
        return make_list(A, r, mk_nil());
      }
      case B_NTH: {
        need(2);
        if (a[0].tag != INT || !is_proper_list(a[1])) fail(E_TYPE);
        if (a[0].i < 0) fail(E_ARG);
        std::vector<Val> xs = list_elems(a[1]);
        if ((uint64_t)a[0].i >= xs.size()) return mk_nil();
        return xs[(size_t)a[0].i];
      }
      case B_PAR: {                                          // (||| n f l1 ... lm), c.7 (L546-589)
        if (n < 3) fail(E_ARITY);
        if (a[0].tag != INT) fail(E_TYPE);
        if (a[1].tag != BUILTIN && a[1].tag != CLOSURE) fail(E_TYPE);
        int64_t cnt = a[0].i;
        if (cnt < 0) fail(E_ARG);
        std::vector<std::vector<Val>> lists;
        for (size_t k = 2; k < n; ++k) {
          if (!is_proper_list(a[k])) fail(E_ARG);
          lists.push_back(list_elems(a[k]));
          if ((int64_t)lists.back().size() < cnt) fail(E_ARG);
        }
        // worker i gets (f l1[i] l2[i] ...) (L562-568); results assembled in order (L584-587)
        std::vector<Val> results;
        for (int64_t i = 0; i < cnt; ++i) {
          std::vector<Val> elems;
          for (auto& l : lists) elems.push_back(l[(size_t)i]);
          results.push_back(apply_fn(a[1], elems, depth));
        }
        return make_list(A, results, mk_nil());
      }
    }
    fail(E_SYNTAX);
  }
};

// one top-level form: (err, steps, value)
struct FormResult { int err; uint64_t steps; std::string printed; };

static FormResult run_form(Session& S, Arena& A, Val form, bool define_mode, bool want_print) {
  Interp I(S, A, define_mode);
  FormResult r{E_OK, 0, std::string()};
  try {
    Val v = I.eval(form, nullptr, 1);                      // top-level eval is depth 1 (c.10)
    r.steps = I.steps;
    if (want_print) print_val(S, v, r.printed);
  } catch (const LispError& e) {
    r.err = e.code;
    r.steps = (e.code == E_FUEL) ? S.fuel + 1 : I.steps;     // c.10
    if (want_print) { r.printed = "#<error "; r.printed += kErrName[e.code]; r.printed += ">"; }
  }
  return r;
}

}  // namespace oracle

// ===================================== C API (ctypes) =================================================
using namespace oracle;

extern "C" {

void* oracle_new(uint32_t max_depth, uint64_t fuel) { return new Session(max_depth, fuel); }
void oracle_delete(void* s) { delete static_cast<Session*>(s); }
void oracle_free(char* p) { std::free(p); }

static char* dup_out(const std::string& s, size_t* len) {
  char* p = (char*)std::malloc(s.size() + 1);
  std::memcpy(p, s.data(), s.size());
  p[s.size()] = 0;
  if (len) *len = s.size();
  return p;
}

// Evaluate definitions sequentially in define mode; allocations persist (L98-101).
// 0 ok; -2 read error (*err_offset); -6 a form failed (*failed_index, *failed_err); that binding is
// not created.
int oracle_define(void* sp, const char* text, size_t len, int64_t* failed_index, int* failed_err,
                  size_t* err_offset) {
  Session& S = *static_cast<Session*>(sp);
  std::string src(text, len);
  std::vector<Val> forms;
  try {
    Reader R(S, S.persistent, src);
    forms = R.all();
  } catch (const ReadError& e) {
    if (err_offset) *err_offset = e.offset;
    return -2;
  }
  for (size_t k = 0; k < forms.size(); ++k) {
    FormResult r = run_form(S, S.persistent, forms[k], true, false);
    if (r.err) {
      if (failed_index) *failed_index = (int64_t)k;
      if (failed_err) *failed_err = r.err;
      return -6;
    }
  }
  return 0;
}

// Evaluate a batch of independent forms (batch mode: the global env is read-only).  Forms are spread
// over `nthreads` std::threads in chunks of 64 -- for timing only; each form is still
// evaluated by one plain recursive walk.  Output (if want_output): one line per form
// "<err>\t<steps>\t<printed>\n" in form order.
int oracle_eval(void* sp, const char* text, size_t len, int nthreads, int want_output, char** out,
                size_t* out_len, double* eval_seconds, uint64_t* total_steps, uint64_t* nforms,
                size_t* err_offset) {
  Session& S = *static_cast<Session*>(sp);
  std::string src(text, len);
  Arena image;
  std::vector<Val> forms;
  try {
    Reader R(S, image, src);
    forms = R.all();
  } catch (const ReadError& e) {
    if (err_offset) *err_offset = e.offset;
    return -2;
  }
  if (nthreads < 1) nthreads = 1;
  std::vector<FormResult> res(forms.size());
  std::atomic<size_t> next{0};
  auto worker = [&]() {
    Arena A;
    for (;;) {
      size_t b = next.fetch_add(64);
      if (b >= forms.size()) break;
      size_t e = std::min(forms.size(), b + 64);
      for (size_t k = b; k < e; ++k) {
        res[k] = run_form(S, A, forms[k], false, want_output != 0);
        A.reset();
      }
    }
  };
  auto t0 = std::chrono::steady_clock::now();
  if (nthreads == 1) {
    worker();
  } else {
    std::vector<std::thread> ts;
    for (int t = 0; t < nthreads; ++t) ts.emplace_back(worker);
    for (auto& t : ts) t.join();
  }
  auto t1 = std::chrono::steady_clock::now();
  if (eval_seconds) *eval_seconds = std::chrono::duration<double>(t1 - t0).count();
  uint64_t tot = 0;
  for (auto& r : res) tot += r.steps;
  if (total_steps) *total_steps = tot;
  if (nforms) *nforms = forms.size();
  if (want_output && out) {
    std::string o;
    for (auto& r : res) {
      o += std::to_string(r.err); o += '\t'; o += std::to_string(r.steps); o += '\t';
      o += r.printed; o += '\n';
    }
    *out = dup_out(o, out_len);
  }
  return 0;
}

// Read and print every datum (printer round-trip pin, c.12).
int oracle_read_print(void* sp, const char* text, size_t len, char** out, size_t* out_len,
                      size_t* err_offset) {
  Session& S = *static_cast<Session*>(sp);
  std::string src(text, len);
  Arena A;
  try {
    Reader R(S, A, src);
    std::vector<Val> forms = R.all();
    std::string o;
    for (Val v : forms) { print_val(S, v, o); o += '\n'; }
    *out = dup_out(o, out_len);
    return 0;
  } catch (const ReadError& e) {
    if (err_offset) *err_offset = e.offset;
    return -2;
  }
}

}  // extern "C"
