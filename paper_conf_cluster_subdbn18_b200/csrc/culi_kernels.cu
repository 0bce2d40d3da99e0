// culi_kernels.cu — sm_100a kernels of libculi.so: image relocation, the eval/apply machine (define and
// batch modes), and result export.  See culi_eval.cuh for the machine's layout and DESIGN.md §5.
#include <cuda_runtime.h>
#include <math.h>
#include <stdint.h>

#include "culi_eval.cuh"

namespace culi {

// ============================================================================================
// stacks
// ============================================================================================
__device__ __forceinline__ uint4* KS(const EvalArgs& A, uint32_t slot, uint32_t i) {
  return A.kst + (size_t)i * A.nslots + slot;
}
__device__ __forceinline__ uint4* VS(const EvalArgs& A, uint32_t slot, uint32_t i) {
  return A.vst + (size_t)i * A.nslots + slot;
}
__device__ __forceinline__ uint4 vpack(V v, uint32_t sym) {
  return make_uint4(lo32(v.w), hi32(v.w), sym, v.t);
}
__device__ __forceinline__ V vunpack(uint4 e) { return mkv(e.w, ((uint64_t)e.y << 32) | e.x); }
__device__ __forceinline__ uint32_t kmeta(uint32_t depth, uint32_t kind, uint32_t count) {
  return depth | (kind << 12) | (count << 16);
}
__device__ __forceinline__ uint32_t kdepth(uint32_t m) { return m & 0xfff; }
__device__ __forceinline__ uint32_t kkind(uint32_t m) { return (m >> 12) & 0xf; }
__device__ __forceinline__ uint32_t kcount(uint32_t m) { return m >> 16; }

// ============================================================================================
// heap access (SoA: tag u8[], word u64[]; PAPER L361-368 node array)
// ============================================================================================
__device__ __forceinline__ uint32_t ntag(const DevHeap& H, uint32_t n) { return H.tag[n]; }
__device__ __forceinline__ uint64_t nword(const DevHeap& H, uint32_t n) { return H.word[n]; }
__device__ __forceinline__ V unbox_loaded(uint32_t n, uint32_t t, uint64_t w) {
  t &= KIND_MASK;
  return mkv(t, is_ref(t) ? (uint64_t)n : w);
}
__device__ __forceinline__ V unbox(const DevHeap& H, uint32_t n) {
  return unbox_loaded(n, ntag(H, n), nword(H, n));
}
__device__ __forceinline__ uint32_t car_of(const DevHeap& H, uint32_t c) { return lo32(nword(H, c)); }
__device__ __forceinline__ uint32_t cdr_of(const DevHeap& H, uint32_t c) { return hi32(nword(H, c)); }

// Warp-aggregated bump allocation (north_star "warp-aggregated atomic bump allocator"; the paper hands
// out "the sequentially next free node", L365-367).  Lanes asking for the same size in the same
// instruction are grouped with __match_any_sync; one atomicAdd per group; lanes get adjacent ranges so
// their stores coalesce.  Returns false when the heap is exhausted.
__device__ __forceinline__ bool heap_alloc(const DevHeap& H, uint32_t n, uint32_t* out) {
  unsigned mask = __activemask();
  unsigned peers = __match_any_sync(mask, n);
  int lane = threadIdx.x & 31;
  int leader = __ffs(peers) - 1;
  unsigned rank = __popc(peers & ((1u << lane) - 1u));
  unsigned long long base = 0;
  if (lane == leader) base = atomicAdd(H.top, (unsigned long long)n * (unsigned)__popc(peers));
  base = __shfl_sync(peers, base, leader);
  unsigned long long mine = base + (unsigned long long)rank * n;
  if (mine + n > H.cap) return false;
  *out = (uint32_t)mine;
  return true;
}

// Store a value into a cons field: references are node indices already; nil/T are nodes 0/1;
// immediates are written into the caller's preallocated box slot.
__device__ __forceinline__ uint32_t box_into(const DevHeap& H, V v, uint32_t slot_node) {
  if (is_ref(v.t)) return (uint32_t)v.w;
  if (v.t == K_NIL) return 0;
  if (v.t == K_T) return 1;
  H.tag[slot_node] = (uint8_t)v.t;
  H.word[slot_node] = v.w;
  return slot_node;
}
__device__ __forceinline__ bool proper_value(const DevHeap& H, V v) {
  return v.t == K_NIL || (v.t == K_CONS && (ntag(H, (uint32_t)v.w) & TAG_PROPER));
}

// ============================================================================================
// environments (§III-B.a; SURVEY c.3)
// ============================================================================================
__device__ __forceinline__ V reserved_value(uint32_t sym) {
  return sym < N_SPECIALS ? mkv(K_SPECIAL, sym) : mkv(K_BUILTIN, sym - N_SPECIALS);
}

// innermost frame first, leftmost binding first, then the global frame; unbound -> the symbol itself
__device__ V lookup(const EvalArgs& A, uint32_t slot, uint32_t sym, uint32_t env) {
  const DevHeap& H = A.H;
  if (sym < N_RESERVED) return reserved_value(sym);
  while (env != 0) {
    if (env & STACK_ENV) {
      uint32_t h = env & ~STACK_ENV;
      uint4 hd = *VS(A, slot, h);
      uint32_t n = hd.z;
      for (uint32_t i = 1; i <= n; ++i) {
        uint4 e = *VS(A, slot, h + i);
        if (e.z == sym) return vunpack(e);
      }
      env = hd.x;
    } else {
      uint64_t hw = nword(H, env);
      uint32_t n = hi32(hw);
      for (uint32_t i = 1; i <= n; ++i) {
        uint64_t bw = nword(H, env + i);
        if (lo32(bw) == sym) return unbox(H, hi32(bw));
      }
      env = lo32(hw);
    }
  }
  uint32_t gt = H.gtag[sym];
  if (gt == K_UNBOUND) return mkv(K_SYM, sym);
  return mkv(gt, H.gword[sym]);
}

// Copy stack frames that a closure captures into the heap (frames are immutable, c.3, so a copy is
// indistinguishable from the original).  Memoised in the stack header (hd.y).
__device__ bool promote(const EvalArgs& A, uint32_t slot, uint32_t env, uint32_t* out) {
  const DevHeap& H = A.H;
  if (!(env & STACK_ENV)) { *out = env; return true; }
  for (;;) {
    uint4 top = *VS(A, slot, env & ~STACK_ENV);
    if (top.y) { *out = top.y; return true; }
    uint32_t e = env;
    for (;;) {
      uint32_t h = e & ~STACK_ENV;
      uint4 hd = *VS(A, slot, h);
      uint32_t p = hd.x;
      uint32_t ph = 0;
      bool ready = true;
      if (p & STACK_ENV) {
        uint32_t pp = VS(A, slot, p & ~STACK_ENV)->y;
        if (pp) ph = pp; else ready = false;
      } else {
        ph = p;
      }
      if (ready) {
        uint32_t n = hd.z, a;
        if (!heap_alloc(H, 1 + 2 * n, &a)) return false;
        H.tag[a] = K_FRAME;
        H.word[a] = pack2(ph, n);
        for (uint32_t i = 0; i < n; ++i) {
          uint4 ent = *VS(A, slot, h + 1 + i);
          uint32_t vn = box_into(H, vunpack(ent), a + 1 + n + i);
          H.tag[a + 1 + i] = K_BIND;
          H.word[a + 1 + i] = pack2(ent.z, vn);
        }
        VS(A, slot, h)->y = a;
        break;
      }
      e = p;
    }
  }
}

__device__ __forceinline__ bool make_closure(const EvalArgs& A, uint32_t slot, uint32_t kind,
                                             uint32_t code, uint32_t env, V* out) {
  uint32_t henv, a;
  if (!promote(A, slot, env, &henv)) return false;
  if (!heap_alloc(A.H, 1, &a)) return false;
  A.H.tag[a] = (uint8_t)kind;
  A.H.word[a] = pack2(code, henv);
  *out = mkv(kind, a);
  return true;
}

// c.5: a parameter list is a proper list of non-reserved symbols
__device__ bool valid_params(const DevHeap& H, uint32_t ps) {
  if (ps == 0) return true;
  uint32_t t = ntag(H, ps);
  if ((t & KIND_MASK) != K_CONS) return false;
  if (!(t & TAG_PROPER)) return false;
  while (ps != 0) {
    uint64_t w = nword(H, ps);
    uint32_t a = lo32(w);
    if ((ntag(H, a) & KIND_MASK) != K_SYM || nword(H, a) < N_RESERVED) return false;
    ps = hi32(w);
  }
  return true;
}
__device__ __forceinline__ bool bindable_node(const DevHeap& H, uint32_t n) {
  return (ntag(H, n) & KIND_MASK) == K_SYM && nword(H, n) >= N_RESERVED;
}

// ============================================================================================
// builtins (SURVEY c.6): args already evaluated at vs[base+1 .. base+cnt];
// order of checks: arity, then types left to right, then compute
// ============================================================================================
__device__ __forceinline__ bool is_num(uint32_t t) { return t == K_INT || t == K_FLOAT; }
__device__ __forceinline__ double as_f64(V v) {
  return v.t == K_INT ? __ll2double_rn((long long)v.w) : __longlong_as_double((long long)v.w);
}
__device__ __forceinline__ V mkf(double d) { return mkv(K_FLOAT, (uint64_t)__double_as_longlong(d)); }
__device__ __forceinline__ V mkb(bool b) { return mkv(b ? K_T : K_NIL, 0); }

__device__ bool eq_values(V a, V b) {
  if (a.t != b.t) return false;
  if (a.t == K_NIL || a.t == K_T) return true;
  return a.w == b.w;    // INT value, FLOAT bits, SYM id, op, or node identity for references
}

// equal: recursive on cons cells; uses the V-stack above vtop as the explicit work stack
__device__ uint8_t equal_values(const EvalArgs& A, uint32_t slot, uint32_t vtop, V a, V b, bool* res) {
  const DevHeap& H = A.H;
  uint32_t sp = vtop;
  for (;;) {
    bool same;
    if (a.t == K_CONS && b.t == K_CONS) {
      uint64_t wa = nword(H, (uint32_t)a.w), wb = nword(H, (uint32_t)b.w);
      if (sp + 2 > A.vcap) return E_OOM;
      *VS(A, slot, sp) = make_uint4(hi32(wa), hi32(wb), 0, 0);     // pending cdr pair
      ++sp;
      a = unbox(H, lo32(wa));
      b = unbox(H, lo32(wb));
      continue;
    }
    if (a.t == K_STR && b.t == K_STR) {
      uint64_t wa = nword(H, (uint32_t)a.w), wb = nword(H, (uint32_t)b.w);
      uint32_t la = hi32(wa), lb = hi32(wb);
      same = la == lb;
      for (uint32_t i = 0; same && i < la; ++i) same = H.strs[lo32(wa) + i] == H.strs[lo32(wb) + i];
    } else {
      same = eq_values(a, b);
    }
    if (!same) { *res = false; return 0; }
    if (sp == vtop) { *res = true; return 0; }
    --sp;
    uint4 pr = *VS(A, slot, sp);
    a = unbox(H, pr.x);
    b = unbox(H, pr.y);
  }
}

__device__ __forceinline__ V arg(const EvalArgs& A, uint32_t slot, uint32_t base, uint32_t i) {
  return vunpack(*VS(A, slot, base + 1 + i));
}

// variadic + - * / : left fold from the first argument (c.6, c.13 #29); INT op INT wraps mod 2^64,
// any FLOAT operand makes that step (and the rest of the fold) f64; IEEE RN, no FMA (c.9)
__device__ uint8_t arith(const EvalArgs& A, uint32_t slot, uint32_t op, uint32_t base, uint32_t cnt,
                         V* out) {
  if ((op == BI_SUB || op == BI_DIV) && cnt == 0) return E_ARITY;
  if (cnt == 0) { *out = mkv(K_INT, op == BI_MUL ? 1 : 0); return 0; }
  bool type_err = false, div0 = false;
  V acc = arg(A, slot, base, 0);
  if (!is_num(acc.t)) type_err = true;
  if (cnt == 1 && (op == BI_SUB || op == BI_DIV)) {
    if (type_err) return E_TYPE;
    if (op == BI_SUB) {
      *out = acc.t == K_INT ? mkv(K_INT, 0ull - acc.w) : mkf(-__longlong_as_double((long long)acc.w));
      return 0;
    }
    V b = acc;                                     // (/ a) = (/ 1 a)
    acc = mkv(K_INT, 1);
    if (b.t == K_INT) {
      if (b.w == 0) return E_DIV0;
      *out = mkv(K_INT, (uint64_t)(1ll / (long long)b.w));
    } else {
      *out = mkf(__ddiv_rn(1.0, as_f64(b)));
    }
    return 0;
  }
  for (uint32_t i = 1; i < cnt; ++i) {
    V b = arg(A, slot, base, i);
    if (!is_num(b.t)) { type_err = true; continue; }
    if (type_err || div0) continue;
    if (acc.t == K_INT && b.t == K_INT) {
      switch (op) {
        case BI_ADD: acc.w = acc.w + b.w; break;
        case BI_SUB: acc.w = acc.w - b.w; break;
        case BI_MUL: acc.w = acc.w * b.w; break;
        default: {
          long long x = (long long)acc.w, y = (long long)b.w;
          if (y == 0) { div0 = true; break; }
          acc.w = (y == -1) ? (0ull - acc.w) : (uint64_t)(x / y);   // INT64_MIN / -1 wraps
        }
      }
    } else {
      double x = as_f64(acc), y = as_f64(b), r;
      switch (op) {
        case BI_ADD: r = __dadd_rn(x, y); break;
        case BI_SUB: r = __dsub_rn(x, y); break;
        case BI_MUL: r = __dmul_rn(x, y); break;
        default: r = __ddiv_rn(x, y); break;
      }
      acc = mkf(r);
    }
  }
  if (type_err) return E_TYPE;
  if (div0) return E_DIV0;
  *out = acc;
  return 0;
}

__device__ uint8_t apply_builtin(const EvalArgs& A, uint32_t slot, uint32_t op, uint32_t base,
                                 uint32_t cnt, uint32_t vtop, V* out) {
  const DevHeap& H = A.H;
  switch (op) {
    case BI_ADD: case BI_SUB: case BI_MUL: case BI_DIV:
      return arith(A, slot, op, base, cnt, out);
    case BI_REM: case BI_MOD: {
      if (cnt != 2) return E_ARITY;
      V a = arg(A, slot, base, 0), b = arg(A, slot, base, 1);
      if (a.t != K_INT || b.t != K_INT) return E_TYPE;
      long long x = (long long)a.w, y = (long long)b.w;
      if (y == 0) return E_DIV0;
      long long r = (y == -1) ? 0 : x % y;
      if (op == BI_MOD && r != 0 && ((r < 0) != (y < 0))) r += y;
      *out = mkv(K_INT, (uint64_t)r);
      return 0;
    }
    case BI_SQRT: case BI_FLOAT: case BI_TRUNC: {
      if (cnt != 1) return E_ARITY;
      V a = arg(A, slot, base, 0);
      if (!is_num(a.t)) return E_TYPE;
      if (op == BI_SQRT) { *out = mkf(__dsqrt_rn(as_f64(a))); return 0; }
      if (op == BI_FLOAT) { *out = mkf(as_f64(a)); return 0; }
      if (a.t == K_INT) { *out = a; return 0; }
      double x = __longlong_as_double((long long)a.w);
      if (isnan(x) || fabs(x) >= 9223372036854775808.0) return E_ARG;
      *out = mkv(K_INT, (uint64_t)__double2ll_rz(x));
      return 0;
    }
    case BI_NUMEQ: case BI_LT: case BI_GT: case BI_LE: case BI_GE: {
      if (cnt != 2) return E_ARITY;
      V a = arg(A, slot, base, 0), b = arg(A, slot, base, 1);
      if (!is_num(a.t) || !is_num(b.t)) return E_TYPE;
      bool r;
      if (a.t == K_INT && b.t == K_INT) {
        long long x = (long long)a.w, y = (long long)b.w;
        r = op == BI_NUMEQ ? x == y : op == BI_LT ? x < y : op == BI_GT ? x > y : op == BI_LE ? x <= y : x >= y;
      } else {
        double x = as_f64(a), y = as_f64(b);
        r = op == BI_NUMEQ ? x == y : op == BI_LT ? x < y : op == BI_GT ? x > y : op == BI_LE ? x <= y : x >= y;
      }
      *out = mkb(r);
      return 0;
    }
    case BI_EQ: {
      if (cnt != 2) return E_ARITY;
      *out = mkb(eq_values(arg(A, slot, base, 0), arg(A, slot, base, 1)));
      return 0;
    }
    case BI_EQUAL: {
      if (cnt != 2) return E_ARITY;
      bool r;
      uint8_t e = equal_values(A, slot, vtop, arg(A, slot, base, 0), arg(A, slot, base, 1), &r);
      if (e) return e;
      *out = mkb(r);
      return 0;
    }
    case BI_NULL: case BI_NOT: case BI_ATOM: case BI_CONSP: case BI_NUMBERP: case BI_SYMBOLP: {
      if (cnt != 1) return E_ARITY;
      uint32_t t = arg(A, slot, base, 0).t;
      bool r = op == BI_NULL || op == BI_NOT ? t == K_NIL
             : op == BI_ATOM ? t != K_CONS
             : op == BI_CONSP ? t == K_CONS
             : op == BI_NUMBERP ? is_num(t)
             : (t == K_SYM || t == K_NIL || t == K_T);
      *out = mkb(r);
      return 0;
    }
    case BI_CONS: {
      if (cnt != 2) return E_ARITY;
      V a = arg(A, slot, base, 0), b = arg(A, slot, base, 1);
      uint32_t c;
      if (!heap_alloc(H, 3, &c)) return E_OOM;
      uint32_t ca = box_into(H, a, c + 1), cd = box_into(H, b, c + 2);
      H.tag[c] = (uint8_t)(K_CONS | (proper_value(H, b) ? TAG_PROPER : 0));
      H.word[c] = pack2(ca, cd);
      *out = mkv(K_CONS, c);
      return 0;
    }
    case BI_CAR: case BI_CDR: {
      if (cnt != 1) return E_ARITY;
      V a = arg(A, slot, base, 0);
      if (a.t == K_NIL) { *out = a; return 0; }
      if (a.t != K_CONS) return E_TYPE;
      uint64_t w = nword(H, (uint32_t)a.w);
      *out = unbox(H, op == BI_CAR ? lo32(w) : hi32(w));
      return 0;
    }
    case BI_LIST: {
      if (cnt == 0) { *out = mkv(K_NIL, 0); return 0; }
      uint32_t c;
      if (!heap_alloc(H, 2 * cnt, &c)) return E_OOM;
      for (uint32_t i = 0; i < cnt; ++i) {
        uint32_t ca = box_into(H, arg(A, slot, base, i), c + cnt + i);
        H.tag[c + i] = K_CONS | TAG_PROPER;
        H.word[c + i] = pack2(ca, i + 1 < cnt ? c + i + 1 : 0);
      }
      *out = mkv(K_CONS, c);
      return 0;
    }
    case BI_LENGTH: {
      if (cnt != 1) return E_ARITY;
      V a = arg(A, slot, base, 0);
      if (!proper_value(H, a)) return E_TYPE;
      uint64_t n = 0;
      for (uint32_t c = a.t == K_NIL ? 0 : (uint32_t)a.w; c != 0; c = cdr_of(H, c)) ++n;
      *out = mkv(K_INT, n);
      return 0;
    }
    case BI_APPEND: {
      if (cnt == 0) { *out = mkv(K_NIL, 0); return 0; }
      uint32_t total = 0;
      for (uint32_t i = 0; i + 1 < cnt; ++i) {
        V a = arg(A, slot, base, i);
        if (!proper_value(H, a)) return E_TYPE;
        for (uint32_t c = a.t == K_NIL ? 0 : (uint32_t)a.w; c != 0; c = cdr_of(H, c)) ++total;
      }
      V last = arg(A, slot, base, cnt - 1);
      if (total == 0) { *out = last; return 0; }
      uint32_t c;
      if (!heap_alloc(H, total + 1, &c)) return E_OOM;
      uint32_t tail = box_into(H, last, c + total);
      uint8_t tg = (uint8_t)(K_CONS | (proper_value(H, last) ? TAG_PROPER : 0));
      uint32_t k = 0;
      for (uint32_t i = 0; i + 1 < cnt; ++i) {
        V a = arg(A, slot, base, i);
        for (uint32_t x = a.t == K_NIL ? 0 : (uint32_t)a.w; x != 0;) {
          uint64_t w = nword(H, x);
          H.tag[c + k] = tg;
          H.word[c + k] = pack2(lo32(w), k + 1 < total ? c + k + 1 : tail);
          ++k;
          x = hi32(w);
        }
      }
      *out = mkv(K_CONS, c);
      return 0;
    }
    case BI_REVERSE: {
      if (cnt != 1) return E_ARITY;
      V a = arg(A, slot, base, 0);
      if (!proper_value(H, a)) return E_TYPE;
      if (a.t == K_NIL) { *out = a; return 0; }
      uint32_t n = 0;
      for (uint32_t x = (uint32_t)a.w; x != 0; x = cdr_of(H, x)) ++n;
      uint32_t c;
      if (!heap_alloc(H, n, &c)) return E_OOM;
      uint32_t k = 0;
      for (uint32_t x = (uint32_t)a.w; x != 0; ++k) {
        uint64_t w = nword(H, x);
        uint32_t j = n - 1 - k;
        H.tag[c + j] = K_CONS | TAG_PROPER;
        H.word[c + j] = pack2(lo32(w), j + 1 < n ? c + j + 1 : 0);
        x = hi32(w);
      }
      *out = mkv(K_CONS, c);
      return 0;
    }
    case BI_NTH: {
      if (cnt != 2) return E_ARITY;
      V i = arg(A, slot, base, 0), l = arg(A, slot, base, 1);
      if (i.t != K_INT || !proper_value(H, l)) return E_TYPE;
      long long k = (long long)i.w;
      if (k < 0) return E_ARG;
      uint32_t x = l.t == K_NIL ? 0 : (uint32_t)l.w;
      for (; k > 0 && x != 0; --k) x = cdr_of(H, x);
      *out = x == 0 ? mkv(K_NIL, 0) : unbox(H, car_of(H, x));
      return 0;
    }
  }
  return E_SYNTAX;
}

// ============================================================================================
// the eval/apply machine
// ============================================================================================
enum Mode : uint32_t { M_EVAL, M_RET, M_HEAD, M_APPLY, M_BODY };
enum KKind : uint32_t { KF_HEAD = 1, KF_ARGS, KF_BODY, KF_IF, KF_LET, KF_DEFINE, KF_MACRO, KF_PAR, KF_DATA };

struct FormOut {
  uint32_t t;
  uint64_t w;
  uint64_t steps;
  uint8_t err;
};

__device__ FormOut eval_form(const EvalArgs& A, uint32_t slot, V root) {
  const DevHeap& H = A.H;
  uint32_t mode = M_EVAL;
  V v = root;
  uint32_t env = 0, d = 1, cur = 0, base = 0, cnt = 0;
  uint32_t sp = 0, vtop = 0;
  uint64_t steps = 0;
  uint8_t err = 0;
  const uint32_t kcap = A.kcap, vcap = A.vcap, maxd = A.max_depth;
  const uint64_t fuel = A.fuel;

#define FAIL(e) do { err = (e); goto done; } while (0)
#define KPUSH(kind, cursor, envv, vsb, depth, count)                                   \
  do {                                                                                 \
    if (sp >= kcap) FAIL(E_OOM);                                                       \
    *KS(A, slot, sp) = make_uint4((cursor), (envv), (vsb), kmeta((depth), (kind), (count))); \
    ++sp;                                                                              \
  } while (0)
#define VPUSH(val, sym)                                                                \
  do {                                                                                 \
    if (vtop >= vcap) FAIL(E_OOM);                                                     \
    *VS(A, slot, vtop) = vpack((val), (sym));                                          \
    ++vtop;                                                                            \
  } while (0)

  for (;;) {
    switch (mode) {
      // ---------------------------------------------------------------- EVAL v in env at depth d
      case M_EVAL: {
        ++steps;                                                  // one canonical step (c.4 step 1)
        if (steps > fuel) FAIL(E_FUEL);
        if (d > maxd) FAIL(E_DEPTH);
        if (v.t == K_SYM) { v = lookup(A, slot, (uint32_t)v.w, env); mode = M_RET; break; }
        if (v.t != K_CONS) { mode = M_RET; break; }               // self-evaluating (L461-462)
        uint32_t x = (uint32_t)v.w;
        uint32_t xt = ntag(H, x);
        uint64_t xw = nword(H, x);
        if (!(xt & TAG_PROPER)) FAIL(E_SYNTAX);
        uint32_t a = lo32(xw);
        cur = hi32(xw);
        uint32_t at = ntag(H, a);
        uint64_t aw = nword(H, a);
        if ((at & KIND_MASK) == K_SYM && aw < N_RESERVED) {
          // the head is a reserved name: its eval step resolves without an env walk (c.5)
          ++steps;
          if (steps > fuel) FAIL(E_FUEL);
          if (d + 1 > maxd) FAIL(E_DEPTH);
          v = reserved_value((uint32_t)aw);
          mode = M_HEAD;
          break;
        }
        KPUSH(KF_HEAD, cur, env, vtop, d, 0);                     // head first (L440-441)
        v = unbox_loaded(a, at, aw);
        d = d + 1;
        break;
      }

      // ---------------------------------------------------------------- head value v, args `cur`
      case M_HEAD: {
        if (v.t == K_SPECIAL) {
          switch ((uint32_t)v.w) {
            case SP_QUOTE: {
              if (cur == 0 || cdr_of(H, cur) != 0) FAIL(E_SYNTAX);
              v = unbox(H, car_of(H, cur));
              mode = M_RET;
              break;
            }
            case SP_IF: {
              if (cur == 0) FAIL(E_SYNTAX);
              uint64_t w0 = nword(H, cur);
              uint32_t c1 = hi32(w0);
              if (c1 == 0) FAIL(E_SYNTAX);
              uint32_t c2 = cdr_of(H, c1);
              if (c2 != 0 && cdr_of(H, c2) != 0) FAIL(E_SYNTAX);
              KPUSH(KF_IF, c1, env, vtop, d, 0);
              v = unbox(H, lo32(w0));
              d = d + 1;
              mode = M_EVAL;
              break;
            }
            case SP_PROGN:
              mode = M_BODY;
              break;
            case SP_LAMBDA: {
              if (cur == 0) FAIL(E_SYNTAX);
              if (!valid_params(H, car_of(H, cur))) FAIL(E_SYNTAX);
              if (!make_closure(A, slot, K_CLOSURE, cur, env, &v)) FAIL(E_OOM);
              mode = M_RET;
              break;
            }
            case SP_LET: {
              if (cur == 0) FAIL(E_SYNTAX);
              uint64_t w0 = nword(H, cur);
              uint32_t bl = lo32(w0), body = hi32(w0);
              if (bl != 0) {                                      // validate every binding first
                uint32_t bt = ntag(H, bl);
                if ((bt & KIND_MASK) != K_CONS || !(bt & TAG_PROPER)) FAIL(E_SYNTAX);
                for (uint32_t c = bl; c != 0; c = cdr_of(H, c)) {
                  uint32_t b = car_of(H, c);
                  uint32_t t = ntag(H, b);
                  if ((t & KIND_MASK) != K_CONS || !(t & TAG_PROPER)) FAIL(E_SYNTAX);
                  uint64_t bw = nword(H, b);
                  if (!bindable_node(H, lo32(bw))) FAIL(E_SYNTAX);
                  uint32_t r = hi32(bw);
                  if (r == 0 || cdr_of(H, r) != 0) FAIL(E_SYNTAX);
                }
              }
              if (bl == 0) { cur = body; mode = M_BODY; break; }
              base = vtop;
              VPUSH(mkv(0, body), 0);                             // header slot (holds body for now)
              KPUSH(KF_LET, bl, env, base, d, 0);
              uint32_t b = car_of(H, bl);
              v = unbox(H, car_of(H, cdr_of(H, b)));              // first init form, outer env
              d = d + 1;
              mode = M_EVAL;
              break;
            }
            case SP_DEFINE: {
              if (!A.define_mode) FAIL(E_DEFINE_IN_BATCH);
              if (cur == 0) FAIL(E_SYNTAX);
              uint64_t w0 = nword(H, cur);
              uint32_t c1 = hi32(w0);
              if (c1 == 0 || cdr_of(H, c1) != 0 || !bindable_node(H, lo32(w0))) FAIL(E_SYNTAX);
              KPUSH(KF_DEFINE, (uint32_t)nword(H, lo32(w0)), env, vtop, d, 0);
              v = unbox(H, car_of(H, c1));
              d = d + 1;
              mode = M_EVAL;
              break;
            }
            case SP_DEFUN:
            case SP_DEFMACRO: {
              uint32_t op = (uint32_t)v.w;
              if (!A.define_mode) FAIL(E_DEFINE_IN_BATCH);
              if (cur == 0) FAIL(E_SYNTAX);
              uint64_t w0 = nword(H, cur);
              uint32_t code = hi32(w0);
              if (code == 0 || !bindable_node(H, lo32(w0)) || !valid_params(H, car_of(H, code)))
                FAIL(E_SYNTAX);
              uint32_t s = (uint32_t)nword(H, lo32(w0));
              V clo;
              if (!make_closure(A, slot, op == SP_DEFUN ? K_CLOSURE : K_MACRO, code, env, &clo))
                FAIL(E_OOM);
              H.gtag[s] = (uint8_t)clo.t;
              H.gword[s] = clo.w;
              v = mkv(K_SYM, s);
              mode = M_RET;
              break;
            }
            default:
              FAIL(E_SYNTAX);
          }
          break;
        }
        if (v.t == K_MACRO) {                                     // c.4 MACRO branch
          uint64_t mw = nword(H, (uint32_t)v.w);
          uint32_t code = lo32(mw), menv = hi32(mw);
          uint64_t cw = nword(H, code);
          uint32_t ps = lo32(cw), body = hi32(cw);
          uint32_t save = vtop;
          uint32_t hdr = vtop;
          VPUSH(mkv(K_FRAME, 0), 0);
          uint32_t n = 0;
          uint32_t a = cur;
          while (ps != 0 && a != 0) {                             // bind params to UNevaluated forms
            uint64_t pw = nword(H, ps), aw = nword(H, a);
            VPUSH(unbox(H, lo32(aw)), (uint32_t)nword(H, lo32(pw)));
            ++n;
            ps = hi32(pw);
            a = hi32(aw);
          }
          if (ps != 0 || a != 0) FAIL(E_ARITY);
          *VS(A, slot, hdr) = make_uint4(menv, 0, n, K_FRAME);
          KPUSH(KF_MACRO, 0, env, save, d, 0);
          env = STACK_ENV | hdr;
          cur = body;
          mode = M_BODY;
          break;
        }
        // data list (L443-444) or (list ...): elements stream into a preallocated contiguous spine
        // (c.14) instead of the V-stack, so arbitrarily wide lists need O(1) stack
        if ((v.t != K_BUILTIN && v.t != K_CLOSURE) || (v.t == K_BUILTIN && v.w == BI_LIST)) {
          bool data = v.t != K_BUILTIN;
          uint32_t n = data ? 1 : 0;
          for (uint32_t c = cur; c != 0; c = cdr_of(H, c)) ++n;
          if (n == 0) { v = mkv(K_NIL, 0); mode = M_RET; break; }
          uint32_t s;
          if (!heap_alloc(H, 2 * n, &s)) FAIL(E_OOM);
          if (data) {
            uint32_t ca = box_into(H, v, s + n);
            H.tag[s] = K_CONS | TAG_PROPER;
            H.word[s] = pack2(ca, n > 1 ? s + 1 : 0);
          }
          if (cur == 0) { v = mkv(K_CONS, s); mode = M_RET; break; }
          base = vtop;
          VPUSH(mkv(0, pack2(s, n)), data ? 1 : 0);            // {spine, n, next index}
          uint64_t w0 = nword(H, cur);
          KPUSH(KF_DATA, hi32(w0), env, base, d, 0);
          v = unbox(H, lo32(w0));
          d = d + 1;
          mode = M_EVAL;
          break;
        }
        // BUILTIN or CLOSURE: evaluate the rest left to right at depth d+1 onto the V-stack
        base = vtop;
        VPUSH(v, 0);
        if (cur == 0) { cnt = 0; mode = M_APPLY; break; }
        {
          uint64_t w0 = nword(H, cur);
          KPUSH(KF_ARGS, hi32(w0), env, base, d, 0);
          v = unbox(H, lo32(w0));
          d = d + 1;
          mode = M_EVAL;
        }
        break;
      }

      // ---------------------------------------------------------------- apply vs[base] to cnt args
      case M_APPLY: {
        V h = vunpack(*VS(A, slot, base));
        if (h.t == K_BUILTIN) {
          if ((uint32_t)h.w == BI_PAR) {                          // (||| n f l1 ... lm), c.7
            if (cnt < 3) FAIL(E_ARITY);
            V nv = arg(A, slot, base, 0), f = arg(A, slot, base, 1);
            if (nv.t != K_INT) FAIL(E_TYPE);
            if (f.t != K_BUILTIN && f.t != K_CLOSURE) FAIL(E_TYPE);
            long long n = (long long)nv.w;
            if (n < 0) FAIL(E_ARG);
            uint32_t m = cnt - 2;
            for (uint32_t j = 0; j < m; ++j) {
              V l = arg(A, slot, base, 2 + j);
              if (!proper_value(H, l)) FAIL(E_ARG);
              uint32_t x = l.t == K_NIL ? 0 : (uint32_t)l.w;
              long long k = 0;
              for (; k < n && x != 0; ++k) x = cdr_of(H, x);
              if (k < n) FAIL(E_ARG);
            }
            if (n == 0) { v = mkv(K_NIL, 0); vtop = base; mode = M_RET; break; }
            uint32_t spine;
            if (!heap_alloc(H, 2 * (uint32_t)n, &spine)) FAIL(E_OOM);
            // state: vs[base] = {spine, n}, vs[base+1] = f, vs[base+2+j] = list cursor j
            for (uint32_t j = 0; j < m; ++j) *VS(A, slot, base + 2 + j) = *VS(A, slot, base + 3 + j);
            *VS(A, slot, base + 1) = vpack(f, 0);
            *VS(A, slot, base) = make_uint4(spine, (uint32_t)n, 0, 0);
            KPUSH(KF_PAR, 0, 0, base, d, m);
            // element 0
            uint32_t eb = base + 2 + m;
            vtop = eb;
            VPUSH(f, 0);
            for (uint32_t j = 0; j < m; ++j) {
              uint4* cj = VS(A, slot, base + 2 + j);
              uint64_t w = nword(H, cj->x);
              VPUSH(unbox(H, lo32(w)), 0);
              cj->x = hi32(w);
            }
            base = eb;
            cnt = m;
            break;                                                // M_APPLY again
          }
          uint8_t e = apply_builtin(A, slot, (uint32_t)h.w, base, cnt, vtop, &v);
          if (e) FAIL(e);
          vtop = base;
          mode = M_RET;
          break;
        }
        if (h.t == K_CLOSURE) {                                   // PAPER L456-460, c.4 CLOSURE
          uint64_t cwd = nword(H, (uint32_t)h.w);
          uint32_t code = lo32(cwd), cenv = hi32(cwd);
          uint64_t codew = nword(H, code);
          uint32_t ps = lo32(codew);
          for (uint32_t i = 0; i < cnt; ++i) {
            if (ps == 0) FAIL(E_ARITY);
            uint64_t pw = nword(H, ps);
            VS(A, slot, base + 1 + i)->z = (uint32_t)nword(H, lo32(pw));
            ps = hi32(pw);
          }
          if (ps != 0) FAIL(E_ARITY);
          *VS(A, slot, base) = make_uint4(cenv, 0, cnt, K_FRAME);
          env = STACK_ENV | base;
          vtop = base + 1 + cnt;
          cur = hi32(codew);
          mode = M_BODY;
          break;
        }
        // data list (L443-444): fresh contiguous list (h v2 ... vn)
        {
          uint32_t n = cnt + 1, c;
          if (!heap_alloc(H, 2 * n, &c)) FAIL(E_OOM);
          for (uint32_t i = 0; i < n; ++i) {
            uint32_t ca = box_into(H, vunpack(*VS(A, slot, base + i)), c + n + i);
            H.tag[c + i] = K_CONS | TAG_PROPER;
            H.word[c + i] = pack2(ca, i + 1 < n ? c + i + 1 : 0);
          }
          v = mkv(K_CONS, c);
          vtop = base;
          mode = M_RET;
        }
        break;
      }

      // ---------------------------------------------------------------- implicit progn of `cur`
      case M_BODY: {
        if (cur == 0) { v = mkv(K_NIL, 0); mode = M_RET; break; }
        uint64_t w0 = nword(H, cur);
        uint32_t nx = hi32(w0);
        if (nx != 0) KPUSH(KF_BODY, nx, env, vtop, d, 0);
        v = unbox(H, lo32(w0));
        d = d + 1;
        mode = M_EVAL;
        break;
      }

      // ---------------------------------------------------------------- return v to the top frame
      case M_RET: {
        if (sp == 0) goto done;
        uint4 k = *KS(A, slot, sp - 1);
        uint32_t kind = kkind(k.w), kd = kdepth(k.w);
        switch (kind) {
          case KF_HEAD:
            --sp;
            cur = k.x;
            env = k.y;
            vtop = k.z;
            d = kd;
            mode = M_HEAD;
            break;
          case KF_ARGS: {
            base = k.z;
            cnt = kcount(k.w);
            vtop = base + 1 + cnt;
            VPUSH(v, 0);
            ++cnt;
            if (k.x != 0) {
              if (cnt >= 0xffff) FAIL(E_OOM);
              uint64_t w0 = nword(H, k.x);
              *KS(A, slot, sp - 1) = make_uint4(hi32(w0), k.y, base, kmeta(kd, KF_ARGS, cnt));
              v = unbox(H, lo32(w0));
              env = k.y;
              d = kd + 1;
              mode = M_EVAL;
            } else {
              --sp;
              d = kd;
              mode = M_APPLY;
            }
            break;
          }
          case KF_BODY: {
            vtop = k.z;
            uint64_t w0 = nword(H, k.x);
            uint32_t nx = hi32(w0);
            if (nx == 0) --sp;
            else KS(A, slot, sp - 1)->x = nx;
            v = unbox(H, lo32(w0));
            env = k.y;
            d = kd + 1;
            mode = M_EVAL;
            break;
          }
          case KF_IF: {
            --sp;
            vtop = k.z;
            env = k.y;
            d = kd + 1;
            uint64_t w1 = nword(H, k.x);
            if (v.t != K_NIL) {
              v = unbox(H, lo32(w1));
              mode = M_EVAL;
            } else if (hi32(w1) != 0) {
              v = unbox(H, car_of(H, hi32(w1)));
              mode = M_EVAL;
            } else {
              v = mkv(K_NIL, 0);
              mode = M_RET;
            }
            break;
          }
          case KF_LET: {
            base = k.z;
            cnt = kcount(k.w);
            uint64_t lw = nword(H, k.x);
            uint32_t sym = (uint32_t)nword(H, car_of(H, lo32(lw)));
            vtop = base + 1 + cnt;
            VPUSH(v, sym);
            ++cnt;
            uint32_t nx = hi32(lw);
            if (nx != 0) {
              if (cnt >= 0xffff) FAIL(E_OOM);
              *KS(A, slot, sp - 1) = make_uint4(nx, k.y, base, kmeta(kd, KF_LET, cnt));
              v = unbox(H, car_of(H, cdr_of(H, car_of(H, nx))));
              env = k.y;
              d = kd + 1;
              mode = M_EVAL;
            } else {
              --sp;
              cur = VS(A, slot, base)->x;                         // body list stored in the header
              *VS(A, slot, base) = make_uint4(k.y, 0, cnt, K_FRAME);
              env = STACK_ENV | base;
              d = kd;
              mode = M_BODY;
            }
            break;
          }
          case KF_DEFINE: {
            --sp;
            H.gtag[k.x] = (uint8_t)v.t;
            H.gword[k.x] = v.w;
            v = mkv(K_SYM, k.x);
            vtop = k.z;
            mode = M_RET;
            break;
          }
          case KF_MACRO: {                                        // evaluate the expansion
            --sp;
            vtop = k.z;
            env = k.y;
            d = kd + 1;
            mode = M_EVAL;
            break;
          }
          case KF_PAR: {                                          // element i finished
            base = k.z;
            uint32_t m = kcount(k.w), i = k.x;
            uint4 st = *VS(A, slot, base);
            uint32_t spine = st.x, n = st.y;
            uint32_t ca = box_into(H, v, spine + n + i);
            H.tag[spine + i] = K_CONS | TAG_PROPER;
            H.word[spine + i] = pack2(ca, i + 1 < n ? spine + i + 1 : 0);
            if (i + 1 == n) {
              --sp;
              v = mkv(K_CONS, spine);
              vtop = base;
              mode = M_RET;
              break;
            }
            KS(A, slot, sp - 1)->x = i + 1;
            V f = vunpack(*VS(A, slot, base + 1));
            uint32_t eb = base + 2 + m;
            vtop = eb;
            VPUSH(f, 0);
            for (uint32_t j = 0; j < m; ++j) {
              uint4* cj = VS(A, slot, base + 2 + j);
              uint64_t w = nword(H, cj->x);
              VPUSH(unbox(H, lo32(w)), 0);
              cj->x = hi32(w);
            }
            base = eb;
            cnt = m;
            d = kd;
            mode = M_APPLY;
            break;
          }
          case KF_DATA: {                                         // next list element arrived
            uint4* st = VS(A, slot, k.z);
            uint4 sv = *st;
            uint32_t s = sv.x, n = sv.y, i = sv.z;
            uint32_t ca = box_into(H, v, s + n + i);
            H.tag[s + i] = K_CONS | TAG_PROPER;
            H.word[s + i] = pack2(ca, i + 1 < n ? s + i + 1 : 0);
            if (k.x != 0) {
              st->z = i + 1;
              uint64_t w0 = nword(H, k.x);
              KS(A, slot, sp - 1)->x = hi32(w0);
              vtop = k.z + 1;
              v = unbox(H, lo32(w0));
              env = k.y;
              d = kd + 1;
              mode = M_EVAL;
            } else {
              --sp;
              vtop = k.z;
              v = mkv(K_CONS, s);
              mode = M_RET;
            }
            break;
          }
          default:
            FAIL(E_SYNTAX);
        }
        break;
      }
    }
  }
done:
#undef FAIL
#undef KPUSH
#undef VPUSH
  FormOut o;
  o.t = v.t;
  o.w = v.w;
  o.steps = steps;
  o.err = err;
  return o;
}

// ============================================================================================
// kernels
// ============================================================================================

// Relocate an uploaded image in place: image-local indices -> heap indices.
__global__ void culi_relocate_kernel(uint8_t* tag, uint64_t* word, uint64_t base, uint64_t n,
                                     uint32_t str_base, uint32_t* roots, uint32_t nroots) {
  uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
    uint64_t g = base + i;
    uint32_t t = tag[g] & KIND_MASK;
    if (t == K_CONS) {
      uint64_t w = word[g];
      uint32_t a = lo32(w), b = hi32(w);
      a = a < IMG_FIRST ? a : (uint32_t)(base + a - IMG_FIRST);
      b = b < IMG_FIRST ? b : (uint32_t)(base + b - IMG_FIRST);
      word[g] = pack2(a, b);
    } else if (t == K_STR) {
      uint64_t w = word[g];
      word[g] = pack2(lo32(w) + str_base, hi32(w));
    }
  }
  for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < nroots; i += stride) {
    uint32_t r = roots[i];
    roots[i] = r < IMG_FIRST ? r : (uint32_t)(base + r - IMG_FIRST);
  }
}

__device__ __forceinline__ void write_result(const EvalArgs& A, uint32_t f, const FormOut& o) {
  A.rtag[f] = o.err ? (uint8_t)K_ERROR : (uint8_t)o.t;
  A.rerr[f] = o.err;
  A.rsteps[f] = o.steps;
  A.rword[f] = o.w;
  if (o.err == E_OOM) atomicExch(&A.flags[0], 1);
}

// Batch mode: one thread per form; each warp takes 32 consecutive forms of the (binned) order.
__global__ void __launch_bounds__(128) culi_eval_kernel(EvalArgs A) {
  uint32_t slot = blockIdx.x * blockDim.x + threadIdx.x;
  int lane = threadIdx.x & 31;
  for (;;) {
    uint32_t b = 0;
    if (lane == 0) b = atomicAdd(A.next, 32u);
    b = __shfl_sync(0xffffffffu, b, 0);
    if (b >= A.nforms) break;
    uint32_t i = b + lane;
    if (i < A.nforms) {
      uint32_t f = A.perm ? A.perm[i] : i;
      V root = unbox(A.H, A.roots[f]);
      FormOut o = eval_form(A, slot, root);
      write_result(A, f, o);
    }
  }
}

// Define mode (culi_define): the forms are evaluated in order by one thread; define/defun/defmacro
// write the global frame; stops at the first error.
__global__ void culi_define_kernel(EvalArgs A) {
  if (blockIdx.x != 0 || threadIdx.x != 0) return;
  for (uint32_t f = 0; f < A.nforms; ++f) {
    V root = unbox(A.H, A.roots[f]);
    FormOut o = eval_form(A, 0, root);
    write_result(A, f, o);
    if (o.err) {
      A.flags[1] = (int)f + 1;
      A.flags[2] = o.err;
      return;
    }
  }
}

// Export: serialize every CONS/STR result into pre-order tokens {word, tag}; the
// record's word becomes offset | count << 32.  Uses the thread's V-stack as the DFS stack.

__global__ void __launch_bounds__(128) culi_export_kernel(ExportArgs X) {
  uint32_t slot = blockIdx.x * blockDim.x + threadIdx.x;
  for (uint32_t f = slot; f < X.nforms; f += X.nslots) {
    uint32_t t = X.rtag[f];
    if (t != K_CONS && t != K_STR) continue;
    uint32_t root = (uint32_t)X.rword[f];
    // pass 1: count tokens
    unsigned long long ntok = 0;
    uint32_t sp = 0;
    uint32_t n = root;
    bool ovf = false;
    for (;;) {
      ++ntok;
      uint32_t nt = X.tag[n] & KIND_MASK;
      if (nt == K_CONS) {
        uint64_t w = X.word[n];
        if (sp >= X.vcap) { ovf = true; break; }
        X.vst[(size_t)sp * X.nslots + slot].x = hi32(w);
        ++sp;
        n = lo32(w);
        continue;
      }
      if (sp == 0) break;
      --sp;
      n = X.vst[(size_t)sp * X.nslots + slot].x;
    }
    if (ovf) { atomicExch(&X.flags[4], 1); continue; }
    unsigned long long off = atomicAdd(X.pcount, ntok);
    if (off + ntok > X.pcap) { atomicExch(&X.flags[3], 1); continue; }
    // pass 2: write tokens
    n = root;
    sp = 0;
    unsigned long long k = off;
    for (;;) {
      uint32_t nt = X.tag[n] & KIND_MASK;
      uint64_t w = X.word[n];
      X.payload[k++] = make_uint4(lo32(w), hi32(w), nt, 0);
      if (nt == K_CONS) {
        X.vst[(size_t)sp * X.nslots + slot].x = hi32(w);
        ++sp;
        n = lo32(w);
        continue;
      }
      if (sp == 0) break;
      --sp;
      n = X.vst[(size_t)sp * X.nslots + slot].x;
    }
    X.rword[f] = (off & 0xffffffffull) | (ntok << 32);
  }
}

// ---- host launch wrappers (called from culi_capi.cu) -------------------------------------------
cudaError_t launch_relocate(cudaStream_t s, uint8_t* tag, uint64_t* word, uint64_t base, uint64_t n,
                            uint32_t str_base, uint32_t* roots, uint32_t nroots, int sms) {
  uint64_t work = n > nroots ? n : nroots;
  uint64_t blocks = (work + 255) / 256;
  if (blocks > (uint64_t)sms * 16) blocks = (uint64_t)sms * 16;
  if (blocks == 0) blocks = 1;
  culi_relocate_kernel<<<(unsigned)blocks, 256, 0, s>>>(tag, word, base, n, str_base, roots, nroots);
  return cudaGetLastError();
}

cudaError_t launch_eval(cudaStream_t s, const EvalArgs& A, uint32_t blocks) {
  culi_eval_kernel<<<blocks, 128, 0, s>>>(A);
  return cudaGetLastError();
}

cudaError_t launch_define(cudaStream_t s, const EvalArgs& A) {
  culi_define_kernel<<<1, 32, 0, s>>>(A);
  return cudaGetLastError();
}

cudaError_t launch_export(cudaStream_t s, const ExportArgs& X, uint32_t blocks) {
  culi_export_kernel<<<blocks, 128, 0, s>>>(X);
  return cudaGetLastError();
}

__global__ void culi_reset_kernel(unsigned long long* top, unsigned long long top_value, uint32_t* next,
                                  unsigned long long* pcount, int* flags) {
  *top = top_value;
  *next = 0;
  *pcount = 0;
  for (int k = 0; k < 8; ++k) flags[k] = 0;
}

cudaError_t launch_reset(cudaStream_t s, unsigned long long* top, unsigned long long top_value,
                         uint32_t* next, unsigned long long* pcount, int* flags) {
  culi_reset_kernel<<<1, 1, 0, s>>>(top, top_value, next, pcount, flags);
  return cudaGetLastError();
}

}  // namespace culi
