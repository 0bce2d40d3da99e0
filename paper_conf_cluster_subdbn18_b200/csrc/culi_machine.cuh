// culi_machine.cuh — the explicit-stack eval/apply machine (device code, sm_100a).
//
// Semantics: SURVEY.md §8(c).4-7 (§III-B.c eval, L383-413 environments, L546-589 |||),
// replayed in exactly the recursive definition's order so that canonical step counts, depths and the
// first error match the oracle.  Design:
//   * control flow is a set of labels joined by gotos — no interpreter `switch` on a mode register;
//   * atoms, symbols and reserved heads are evaluated inline where they occur, so only a nested *list*
//     costs a continuation; ≤2-argument builtins whose arguments are all atoms/symbols are computed in
//     registers without touching the V-stack (e.g. (- n 1), (< n 2));
//   * K-stack (continuations, uint4) and V-stack (values / frame bindings, uint4) in HBM, level-major
//     across threads so lock-step warps coalesce; the top continuation lives in registers with a dirty
//     bit, so a continuation pushed and popped without an intervening push never touches memory;
//   * environment references: heap frame node index, or STACK_ENV | n << 16 | vs_index for a frame on
//     the thread's V-stack (n bindings), so a hit in the innermost frame costs one load;
//   * the global frame (direct-indexed by symbol id) and the persistent code segment are staged in
//     shared memory per block; special-form syntax of reader-produced lists is
//     validated once on the host (TAG_VALID).
#pragma once
#include <cuda_runtime.h>
#include <math.h>
#include <stdint.h>

#include "culi_eval.cuh"

namespace culi {

#ifndef CULI_COLD
#define CULI_COLD __noinline__
#endif

extern __shared__ __align__(16) uint4 culi_smem[];   // [code nodes][global words][global tags]

// Cold (out-of-line) helpers take Ctx by value: passing the hot path's Ctx by reference would make it
// escape to memory, and every launch constant would then cost a local + a generic load (measured).
struct Ctx {
  const EvalArgs* A;         // the launch's constants (a __grid_constant__ kernel parameter)
  uint4* kb;                 // &kst[slot]   (entry i at kb + i * nslots)
  uint4* vb;                 // &vst[slot]
};

// entry i of this thread's stacks: one IMAD.WIDE.U32 with the precomputed byte stride (nslots * 16)
__device__ __forceinline__ uint4* KS(const Ctx& C, uint32_t i) {
  return reinterpret_cast<uint4*>(reinterpret_cast<char*>(C.kb) + (size_t)i * C.A->stride);
}
__device__ __forceinline__ uint4* VS(const Ctx& C, uint32_t i) {
  return reinterpret_cast<uint4*>(reinterpret_cast<char*>(C.vb) + (size_t)i * C.A->stride);
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

constexpr uint32_t ENV_IDX_MASK = 0xffffu;
__device__ __forceinline__ uint32_t stack_env(uint32_t idx, uint32_t n) {
  return STACK_ENV | (n << 16) | idx;
}
// reference kinds: STR, CONS, CLOSURE, MACRO (value word = node index)
constexpr uint32_t REF_MASK = (1u << K_STR) | (1u << K_CONS) | (1u << K_CLOSURE) | (1u << K_MACRO);
__device__ __forceinline__ bool is_ref_k(uint32_t k) { return (REF_MASK >> k) & 1u; }

// ---- staged shared memory -----------------------------------------------------------------------------
__device__ __forceinline__ const uint64_t* sm_gword(const Ctx& C) {
#if CULI_STAGE_CODE
  return reinterpret_cast<const uint64_t*>(culi_smem + C.A->code_n);
#else
  return reinterpret_cast<const uint64_t*>(culi_smem);            // no code segment staged (code_n = 0)
#endif
}
__device__ __forceinline__ const uint8_t* sm_gtag(const Ctx& C) {
  return reinterpret_cast<const uint8_t*>(sm_gword(C) + C.A->gst);
}

// ---- heap access (16-byte nodes {word, tag}, culi_internal.h) ------------------------------
// CULI_STAGE_CODE=1 serves the persistent code segment from shared memory.  Measured on C2 (round 1):
// the range check makes every node load execute both paths predicated (~25 % of all instructions),
// which costs more than the L1 hits it replaces, so it is off by default; the global frame (one lookup
// site) stays staged.
#ifndef CULI_STAGE_CODE
#define CULI_STAGE_CODE 0
#endif
__device__ __forceinline__ void ldnode(const Ctx& C, uint32_t n, uint32_t& t, uint64_t& w) {
#if CULI_STAGE_CODE
  uint32_t r = n - C.A->code_lo;
  if (r < C.A->code_n) {
    uint4 q = culi_smem[r];
    t = q.z;
    w = ((uint64_t)q.y << 32) | q.x;
    return;
  }
#endif
  const uint4 q = *reinterpret_cast<const uint4*>(C.A->H.tag.p + n);   // one 16-byte load per node
  t = q.z & 0xffu;                          // (flag bits PROPER / VALID / LEN: every consumer masks)
  w = ((uint64_t)q.y << 32) | q.x;
}
__device__ __forceinline__ uint64_t nword(const Ctx& C, uint32_t n) {
#if CULI_STAGE_CODE
  uint32_t r = n - C.A->code_lo;
  if (r < C.A->code_n) { uint2 q = *reinterpret_cast<const uint2*>(&culi_smem[r]); return ((uint64_t)q.y << 32) | q.x; }
#endif
  return C.A->H.word[n];
}
__device__ __forceinline__ uint32_t ntag(const Ctx& C, uint32_t n) {
#if CULI_STAGE_CODE
  uint32_t r = n - C.A->code_lo;
  if (r < C.A->code_n) return culi_smem[r].z;
#endif
  return C.A->H.tag[n];
}
__device__ __forceinline__ V unbox_loaded(uint32_t n, uint32_t t, uint64_t w) {
  t &= KIND_MASK;
  return mkv(t, is_ref_k(t) ? (uint64_t)n : w);
}
__device__ __forceinline__ V unbox(const Ctx& C, uint32_t n) {
  uint32_t t;
  uint64_t w;
  ldnode(C, n, t, w);
  return unbox_loaded(n, t, w);
}
__device__ __forceinline__ uint32_t car_of(const Ctx& C, uint32_t c) { return lo32(nword(C, c)); }
__device__ __forceinline__ uint32_t cdr_of(const Ctx& C, uint32_t c) { return hi32(nword(C, c)); }

#ifndef CULI_NEST_TRACE
#define CULI_NEST_TRACE 0
#endif
__device__ __forceinline__ unsigned long long gtime_trace() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}
#if CULI_NEST_TRACE
// debug (-DCULI_NEST_TRACE=1): [0] first claim, [1] last element done, [2] owner resumed, [3] owner suspended,
// [4] claims, [5] first thread started, [6] owner at DATA_START, [7] owner after the cell count (globaltimer)
__device__ unsigned long long culi_nest_trace[8];
__host__ inline int culi_nest_trace_read(unsigned long long* out) {
  return cudaMemcpyFromSymbol(out, culi_nest_trace, sizeof(culi_nest_trace)) == cudaSuccess ? 0 : 1;
}
__host__ inline int culi_nest_trace_reset() {
  unsigned long long z[8] = {~0ull, 0, 0, ~0ull, 0, ~0ull, 0, 0};
  return cudaMemcpyToSymbol(culi_nest_trace, z, sizeof(z)) == cudaSuccess ? 0 : 1;
}
#define NTRACE_MIN(k) atomicMin(&culi_nest_trace[k], gtime_trace())
#define NTRACE_MAX(k) atomicMax(&culi_nest_trace[k], gtime_trace())
#define NTRACE_ADD(k, v) atomicAdd(&culi_nest_trace[k], (unsigned long long)(v))
#else
#define NTRACE_MIN(k) do { } while (0)
#define NTRACE_MAX(k) do { } while (0)
#define NTRACE_ADD(k, v) do { } while (0)
#endif

// Length of the cdr chain from c (the count loop of a data list / list).  Reader spines are contiguous
// (c.14), so the next 16 cells are loaded before their links are checked (branch-free, so all loads are in
// flight together: one L2 round trip per 16 cells instead of one per cell); a link that leaves the run
// restarts the scan there, so exactly the same chain is walked.  Out of line: its registers stay out of
// the eval loop's allocation.
__device__ CULI_COLD uint32_t chain_length(Ctx C, uint32_t c) {
  uint32_t n = 0;
  const uint64_t cap = C.A->H.cap;
  const Node* nodes = C.A->H.tag.p;
  while (c != 0) {
    if ((uint64_t)c + 32 > cap) { ++n; c = cdr_of(C, c); continue; }
    // 32 cells per round trip: the cdr halves of 32 nodes, links checked afterwards (all loads in flight)
    uint32_t q[32];
#pragma unroll
    for (int k = 0; k < 32; ++k) q[k] = reinterpret_cast<const uint32_t*>(nodes + c + k)[1];
    uint32_t brk = 0, nx = c + 32;
#pragma unroll
    for (int k = 31; k >= 0; --k)
      if (q[k] != c + k + 1) { brk |= 1u << k; nx = q[k]; }       // the lowest break wins
    n += brk ? __ffs(brk) : 32;
    c = nx;
  }
  return n;
}

// Warp-aggregated bump allocation (north_star; "the sequentially next free node"):
// lanes asking for the same size in the same instruction share one allocation (__match_any_sync) and
// receive adjacent ranges, so their node stores coalesce.  Small requests come from a per-warp chunk in
// shared memory (one shared atomic; the global bump pointer is touched once per ALLOC_CHUNK nodes), so
// allocation-heavy batches (C4's macro expansions) do not serialise on one global counter.  The chunk
// word packs next | end << 32 (heap indices are < 2^31); a request that overflows the chunk takes a fresh
// one from the global pointer and installs it with one exchange — no retry loop, so nothing spins
// between the two collectives.  Every kernel that allocates zeroes culi_alloc first.
#ifndef CULI_ALLOC_CHUNK
#define CULI_ALLOC_CHUNK 512
#endif
constexpr uint32_t ALLOC_CHUNK = CULI_ALLOC_CHUNK;   // 0: every request goes to the global pointer
__shared__ unsigned long long culi_alloc[4];
__device__ __forceinline__ void alloc_init() {
  if ((threadIdx.x & 31) == 0 && threadIdx.x < 128) culi_alloc[threadIdx.x >> 5] = 0;
}
// CHUNK = false (the warp-voting kernel's own sites): every request goes to the global pointer.  Measured
// on C4 (262,144 macro forms whose diverged lanes allocate one at a time): without the chunk code the
// voting kernel is smaller and faster, while C2 / C5 gain from the chunks (tools/ab.sh).
template <bool CHUNK = true>
__device__ __forceinline__ unsigned long long alloc_range(const DevHeap& H, unsigned long long need) {
  if (!CHUNK || need > ALLOC_CHUNK / 4) return atomicAdd(H.top, need);
  unsigned long long* s = &culi_alloc[threadIdx.x >> 5];
  unsigned long long old = atomicAdd(s, need);
  unsigned long long next = old & 0xffffffffull, end = old >> 32;
  if (next + need <= end) return next;
  unsigned long long b = atomicAdd(H.top, (unsigned long long)ALLOC_CHUNK);
  if (b + ALLOC_CHUNK <= H.cap) atomicExch(s, ((b + ALLOC_CHUNK) << 32) | (b + need));
  return b;
}
template <bool CHUNK = true>
__device__ __forceinline__ bool heap_alloc(const DevHeap& H, uint32_t n, uint32_t* out) {
  unsigned mask = __activemask();
  // (& mask: a lane group of another call converged onto this instruction must not leak into the result,
  // see try_split)
  unsigned peers = __match_any_sync(mask, n) & mask;
  int lane = threadIdx.x & 31;
  int leader = __ffs(peers) - 1;
  unsigned rank = __popc(peers & ((1u << lane) - 1u));
  unsigned long long base = 0;
  if (lane == leader) base = alloc_range<CHUNK>(H, (unsigned long long)n * (unsigned)__popc(peers));
  base = __shfl_sync(peers, base, leader);
  unsigned long long mine = base + (unsigned long long)rank * n;
  if (mine + n > H.cap) return false;
  *out = (uint32_t)mine;
  return true;
}

// store a value into a cons field: references are node indices; nil/T are nodes 0/1; immediates go to
// the caller's preallocated box slot
__device__ __forceinline__ uint32_t box_into(const DevHeap& H, V v, uint32_t slot_node) {
  if (is_ref_k(v.t)) return (uint32_t)v.w;
  if (v.t == K_NIL) return 0;
  if (v.t == K_T) return 1;
  H.tag[slot_node] = (uint8_t)v.t;
  H.word[slot_node] = v.w;
  return slot_node;
}
__device__ __forceinline__ bool proper_value(const Ctx& C, V v) {
  return v.t == K_NIL || (v.t == K_CONS && (ntag(C, (uint32_t)v.w) & TAG_PROPER));
}

// ---- environments (§III-B.a; SURVEY c.3) ------------------------------------------------
__device__ __forceinline__ V reserved_value(uint32_t sym) {
  return sym < N_SPECIALS ? mkv(K_SPECIAL, sym) : mkv(K_BUILTIN, sym - N_SPECIALS);
}
// symbols beyond the staged part of the global frame (and define mode, which stages nothing)
__device__ CULI_COLD V global_value_hbm(Ctx C, uint32_t sym) {
  uint32_t gt = C.A->H.gtag[sym];
  if (gt == K_UNBOUND) return mkv(K_SYM, sym);
  return mkv(gt, C.A->H.gword[sym]);
}
__device__ __forceinline__ V global_value(const Ctx& C, uint32_t sym) {
  if (__builtin_expect(sym >= C.A->gst, 0)) return global_value_hbm(C, sym);
  uint32_t gt = sm_gtag(C)[sym];
  uint64_t gw = sm_gword(C)[sym];
  if (gt == K_UNBOUND) return mkv(K_SYM, sym);
  return mkv(gt, gw);
}

// full walk: innermost frame first, leftmost binding first, then the global frame; unbound -> itself
__device__ CULI_COLD V lookup_slow(Ctx C, uint32_t sym, uint32_t env) {
  while (env != 0) {
    if (env & STACK_ENV) {
      uint32_t h = env & ENV_IDX_MASK, n = (env >> 16) & 0x7fffu;
      for (uint32_t i = 1; i <= n; ++i) {
        uint4 e = *VS(C, h + i);
        if (e.z == sym) return vunpack(e);
      }
      env = VS(C, h)->x;
    } else {
      uint64_t hw = nword(C, env);
      uint32_t n = hi32(hw);
      for (uint32_t i = 1; i <= n; ++i) {
        uint64_t bw = nword(C, env + i);
        if (lo32(bw) == sym) return unbox(C, hi32(bw));
      }
      env = lo32(hw);
    }
  }
  return global_value(C, sym);
}

// fast path: reserved names; the innermost stack frame's first binding; a one-binding stack frame
// whose parent is the global frame (both loads issued together)
__device__ __forceinline__ V lookup(const Ctx& C, uint32_t sym, uint32_t env) {
  if (sym < N_RESERVED) return reserved_value(sym);
  if (env == 0) return global_value(C, sym);
  if (env & STACK_ENV) {
    uint32_t h = env & ENV_IDX_MASK, n = (env >> 16) & 0x7fffu;
    uint4 e = make_uint4(0, 0, 0xffffffffu, 0);
    if (n >= 1) e = *VS(C, h + 1);
    uint32_t parent = VS(C, h)->x;
    if (n >= 1 && e.z == sym) return vunpack(e);
    if (n <= 1 && parent == 0) return global_value(C, sym);

  }
  return lookup_slow(C, sym, env);
}

// Copy the stack frames a closure captures into the heap (frames are immutable, c.3, so a copy is
// indistinguishable from the original).  Memoised in the stack header's .y field.
__device__ CULI_COLD bool promote(Ctx C, uint32_t env, uint32_t* out) {
  const DevHeap& H = C.A->H;
  if (!(env & STACK_ENV)) { *out = env; return true; }
  for (;;) {
    uint32_t topp = VS(C, env & ENV_IDX_MASK)->y;
    if (topp) { *out = topp; return true; }
    uint32_t e = env;
    for (;;) {
      uint32_t h = e & ENV_IDX_MASK;
      uint4 hd = *VS(C, h);
      uint32_t p = hd.x, ph = 0;
      bool ready = true;
      if (p & STACK_ENV) {
        uint32_t pp = VS(C, p & ENV_IDX_MASK)->y;
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
          uint4 ent = *VS(C, h + 1 + i);
          uint32_t vn = box_into(H, vunpack(ent), a + 1 + n + i);
          H.tag[a + 1 + i] = K_BIND;
          H.word[a + 1 + i] = pack2(ent.z, vn);
        }
        VS(C, h)->y = a;
        break;
      }
      e = p;
    }
  }
}

// A closure / macro is three nodes: {kind: code | env << 32}, {K_AUX: nparams | first param << 32} and
// {K_AUX: body | params << 32}, so a call reads all it needs with three independent loads
// (code = the cons (params . body); env = heap frame or 0).
__device__ CULI_COLD bool make_closure(Ctx C, uint32_t kind, uint32_t code, uint32_t env,
                                          V* out) {
  uint32_t henv, a;
  if (!promote(C, env, &henv)) return false;
  uint32_t np = 0, first = 0;
  for (uint32_t p = car_of(C, code); p != 0; p = cdr_of(C, p)) {
    if (np == 0) first = (uint32_t)nword(C, car_of(C, p));
    ++np;
  }
  if (!heap_alloc(C.A->H, 3, &a)) return false;
  C.A->H.tag[a] = (uint8_t)kind;
  C.A->H.word[a] = pack2(code, henv);
  C.A->H.tag[a + 1] = K_AUX;
  C.A->H.word[a + 1] = pack2(np, first);
  C.A->H.tag[a + 2] = K_AUX;                            // body list | parameter list
  C.A->H.word[a + 2] = pack2(cdr_of(C, code), car_of(C, code));
  *out = mkv(kind, a);
  return true;
}

// (setq s v) after v was evaluated (R7): the innermost, leftmost binding of s in env; else the global.
// In a batch, globals and frames made while defining (heap index < pmark) are read-only.
__device__ CULI_COLD uint8_t setq_store(Ctx C, uint32_t sym, uint32_t env, V v) {
  const DevHeap& H = C.A->H;
  while (env != 0) {
    if (env & STACK_ENV) {                                      // (frames are in the heap when mut is set)
      uint32_t h = env & ENV_IDX_MASK, n = (env >> 16) & 0x7fffu;
      for (uint32_t i = 1; i <= n; ++i) {
        uint4* e = VS(C, h + i);
        if (e->z == sym) { *e = vpack(v, sym); return 0; }
      }
      env = VS(C, h)->x;
    } else {
      uint64_t hw = nword(C, env);
      uint32_t n = hi32(hw);
      for (uint32_t i = 1; i <= n; ++i) {
        uint64_t bw = nword(C, env + i);
        if (lo32(bw) != sym) continue;
        if (!C.A->define_mode && env < C.A->pmark) return E_DEFINE_IN_BATCH;
        uint32_t vn = box_into(H, v, env + n + i);              // the binding's own value slot
        H.word[env + i] = pack2(sym, vn);
        return 0;
      }
      env = lo32(hw);
    }
  }
  if (!C.A->define_mode) return E_DEFINE_IN_BATCH;
  H.gtag[sym] = (uint8_t)v.t;
  H.gword[sym] = v.w;
  return 0;
}

// c.5: a parameter list is a proper list of non-reserved symbols
__device__ CULI_COLD bool valid_params(Ctx C, uint32_t ps) {
  if (ps == 0) return true;
  uint32_t t = ntag(C, ps);
  if ((t & KIND_MASK) != K_CONS || !(t & TAG_PROPER)) return false;
  while (ps != 0) {
    uint64_t w = nword(C, ps);
    uint32_t at;
    uint64_t aw;
    ldnode(C, lo32(w), at, aw);
    if ((at & KIND_MASK) != K_SYM || aw < N_RESERVED) return false;
    ps = hi32(w);
  }
  return true;
}
__device__ __forceinline__ bool bindable_node(const Ctx& C, uint32_t n) {
  uint32_t t;
  uint64_t w;
  ldnode(C, n, t, w);
  return (t & KIND_MASK) == K_SYM && w >= N_RESERVED;
}

// ---- builtins (SURVEY c.6): arity, then types left to right, then compute --------------------------
__device__ __forceinline__ bool is_num(uint32_t t) { return t == K_INT || t == K_FLOAT; }
__device__ __forceinline__ double as_f64(V v) {
  return v.t == K_INT ? __ll2double_rn((long long)v.w) : __longlong_as_double((long long)v.w);
}
__device__ __forceinline__ V mkf(double d) { return mkv(K_FLOAT, (uint64_t)__double_as_longlong(d)); }
__device__ __forceinline__ V mkb(bool b) { return mkv(b ? K_T : K_NIL, 0); }
__device__ __forceinline__ V arg(const Ctx& C, uint32_t base, uint32_t i) {
  return vunpack(*VS(C, base + 1 + i));
}
__device__ __forceinline__ bool eq_values(V a, V b) {
  if (a.t != b.t) return false;
  if (a.t == K_NIL || a.t == K_T) return true;
  return a.w == b.w;   // INT value, FLOAT bits, SYM id, op, or node identity for references
}

// one step of a numeric fold (types already checked); returns false on integer division by zero
__device__ CULI_COLD bool fold_float(uint32_t op, V& acc, V b) {
  double x = as_f64(acc), y = as_f64(b), r;
  switch (op) {
    case BI_ADD: r = __dadd_rn(x, y); break;
    case BI_SUB: r = __dsub_rn(x, y); break;
    case BI_MUL: r = __dmul_rn(x, y); break;
    default: r = __ddiv_rn(x, y); break;
  }
  acc = mkf(r);
  return true;
}
__device__ __forceinline__ bool fold_step(uint32_t op, V& acc, V b) {
  if (acc.t == K_INT && b.t == K_INT) {
    switch (op) {
      case BI_ADD: acc.w = acc.w + b.w; return true;
      case BI_SUB: acc.w = acc.w - b.w; return true;
      case BI_MUL: acc.w = acc.w * b.w; return true;
      default: {
        long long x = (long long)acc.w, y = (long long)b.w;
        if (y == 0) return false;
        acc.w = (y == -1) ? (0ull - acc.w) : (uint64_t)(x / y);   // INT64_MIN / -1 wraps
        return true;
      }
    }
  }
  return fold_float(op, acc, b);
}
__device__ __forceinline__ bool cmp_values(uint32_t op, V a, V b) {
  if (a.t == K_INT && b.t == K_INT) {
    long long x = (long long)a.w, y = (long long)b.w;
    return op == BI_NUMEQ ? x == y : op == BI_LT ? x < y : op == BI_GT ? x > y : op == BI_LE ? x <= y : x >= y;
  }
  double x = as_f64(a), y = as_f64(b);
  return op == BI_NUMEQ ? x == y : op == BI_LT ? x < y : op == BI_GT ? x > y : op == BI_LE ? x <= y : x >= y;
}

// Builtins that the register fast path handles when they get at most two arguments.
constexpr uint64_t FAST_OPS =
    (1ull << BI_ADD) | (1ull << BI_SUB) | (1ull << BI_MUL) | (1ull << BI_DIV) | (1ull << BI_REM) |
    (1ull << BI_MOD) | (1ull << BI_NUMEQ) | (1ull << BI_LT) | (1ull << BI_GT) | (1ull << BI_LE) |
    (1ull << BI_GE) | (1ull << BI_EQ) | (1ull << BI_NULL) | (1ull << BI_NOT) | (1ull << BI_ATOM) |
    (1ull << BI_CONSP) | (1ull << BI_NUMBERP) | (1ull << BI_SYMBOLP) | (1ull << BI_CAR) | (1ull << BI_CDR);

// (op a0 [a1]) with argc <= 2 evaluated arguments in registers; same checks as the general path.  Every
// case; out of line (fast2 below inlines only the common ones, to keep the machine's hot code small).
__device__ CULI_COLD uint8_t fast2_full(Ctx C, uint32_t op, uint32_t argc, V a0, V a1, V* out) {
  switch (op) {
    case BI_ADD: case BI_SUB: case BI_MUL: case BI_DIV: {
      if (argc == 0) {
        if (op == BI_SUB || op == BI_DIV) return E_ARITY;
        *out = mkv(K_INT, op == BI_MUL ? 1 : 0);
        return 0;
      }
      if (!is_num(a0.t) || (argc == 2 && !is_num(a1.t))) return E_TYPE;
      if (argc == 1) {
        if (op == BI_SUB) {
          *out = a0.t == K_INT ? mkv(K_INT, 0ull - a0.w) : mkf(-__longlong_as_double((long long)a0.w));
          return 0;
        }
        if (op != BI_DIV) { *out = a0; return 0; }
        a1 = a0;                                     // (/ a) = (/ 1 a)
        a0 = mkv(K_INT, 1);
      }
      if (!fold_step(op, a0, a1)) return E_DIV0;
      *out = a0;
      return 0;
    }
    case BI_REM: case BI_MOD: {
      if (argc != 2) return E_ARITY;
      if (a0.t != K_INT || a1.t != K_INT) return E_TYPE;
      long long x = (long long)a0.w, y = (long long)a1.w;
      if (y == 0) return E_DIV0;
      long long r = (y == -1) ? 0 : x % y;
      if (op == BI_MOD && r != 0 && ((r < 0) != (y < 0))) r += y;
      *out = mkv(K_INT, (uint64_t)r);
      return 0;
    }
    case BI_NUMEQ: case BI_LT: case BI_GT: case BI_LE: case BI_GE:
      if (argc != 2) return E_ARITY;
      if (!is_num(a0.t) || !is_num(a1.t)) return E_TYPE;
      *out = mkb(cmp_values(op, a0, a1));
      return 0;
    case BI_EQ:
      if (argc != 2) return E_ARITY;
      *out = mkb(eq_values(a0, a1));
      return 0;
    case BI_CAR: case BI_CDR: {
      if (argc != 1) return E_ARITY;
      if (a0.t == K_NIL) { *out = a0; return 0; }
      if (a0.t != K_CONS) return E_TYPE;
      uint64_t w = nword(C, (uint32_t)a0.w);
      *out = unbox(C, op == BI_CAR ? lo32(w) : hi32(w));
      return 0;
    }
    default: {                                       // one-argument predicates
      if (argc != 1) return E_ARITY;
      uint32_t t = a0.t;
      bool r = op == BI_NULL || op == BI_NOT ? t == K_NIL
             : op == BI_ATOM ? t != K_CONS
             : op == BI_CONSP ? t == K_CONS
             : op == BI_NUMBERP ? is_num(t)
             : (t == K_SYM || t == K_NIL || t == K_T);
      *out = mkb(r);
      return 0;
    }
  }
}

// Inline front of fast2_full: int64 (+ - *) and comparisons of two INTs, null/not, car/cdr of a cons.
// Instruction fetch is the machine's top stall: one compact copy per call site.
__device__ __forceinline__ uint8_t fast2(const Ctx& C, uint32_t op, uint32_t argc, V a0, V a1, V* out) {
  if (argc == 2 && a0.t == K_INT && a1.t == K_INT) {
    uint64_t x = a0.w, y = a1.w;
    if (op <= BI_MUL && op != BI_DIV) {
      out->t = K_INT;
      out->w = op == BI_ADD ? x + y : op == BI_SUB ? x - y : x * y;
      return 0;
    }
    if (op >= BI_NUMEQ && op <= BI_GE) {
      long long sx = (long long)x, sy = (long long)y;
      bool lt = sx < sy, eq = sx == sy;
      bool r = op == BI_NUMEQ ? eq : op == BI_LT ? lt : op == BI_GT ? !(lt || eq) : op == BI_LE ? (lt || eq) : !lt;
      *out = mkb(r);
      return 0;
    }
  }
  if (argc == 1) {
    if (op == BI_NULL || op == BI_NOT) { *out = mkb(a0.t == K_NIL); return 0; }
    if ((op == BI_CAR || op == BI_CDR) && a0.t == K_CONS) {
      uint64_t w = nword(C, (uint32_t)a0.w);
      *out = unbox(C, op == BI_CAR ? lo32(w) : hi32(w));
      return 0;
    }
  }
  return fast2_full(C, op, argc, a0, a1, out);
}

// equal: recursive on cons cells, with the V-stack above vtop as the explicit work stack
__device__ CULI_COLD uint8_t equal_values(Ctx C, uint32_t vtop, V a, V b, bool* res) {
  uint32_t sp = vtop;
  for (;;) {
    bool same;
    if (a.t == K_CONS && b.t == K_CONS) {
      uint64_t wa = nword(C, (uint32_t)a.w), wb = nword(C, (uint32_t)b.w);
      if (sp + 1 >= C.A->vcap) return E_OOM;
      *VS(C, sp) = make_uint4(hi32(wa), hi32(wb), 0, 0);
      ++sp;
      a = unbox(C, lo32(wa));
      b = unbox(C, lo32(wb));
      continue;
    }
    if (a.t == K_STR && b.t == K_STR) {
      uint64_t wa = nword(C, (uint32_t)a.w), wb = nword(C, (uint32_t)b.w);
      uint32_t la = hi32(wa), lb = hi32(wb);
      same = la == lb;
      for (uint32_t i = 0; same && i < la; ++i) same = C.A->H.strs[lo32(wa) + i] == C.A->H.strs[lo32(wb) + i];
    } else {
      same = eq_values(a, b);
    }
    if (!same) { *res = false; return 0; }
    if (sp == vtop) { *res = true; return 0; }
    --sp;
    uint4 pr = *VS(C, sp);
    a = unbox(C, pr.x);
    b = unbox(C, pr.y);
  }
}

// general builtin application over vs[base+1 .. base+cnt] (any arity)
template <bool CHUNK = true>
__device__ CULI_COLD uint8_t apply_builtin(Ctx C, uint32_t op, uint32_t base, uint32_t cnt,
                                              uint32_t vtop, V* out) {
  const DevHeap& H = C.A->H;
  if (((FAST_OPS >> op) & 1) && cnt <= 2) {
    V a0 = cnt > 0 ? arg(C, base, 0) : mkv(K_NIL, 0), a1 = cnt > 1 ? arg(C, base, 1) : mkv(K_NIL, 0);
    return fast2_full(C, op, cnt, a0, a1, out);
  }
  switch (op) {
    case BI_ADD: case BI_SUB: case BI_MUL: case BI_DIV: {       // cnt >= 3: left fold (c.13 #29)
      bool type_err = false, div0 = false;
      for (uint32_t i = 0; i < cnt; ++i) type_err |= !is_num(arg(C, base, i).t);
      if (type_err) return E_TYPE;
      V acc = arg(C, base, 0);
      for (uint32_t i = 1; i < cnt && !div0; ++i) div0 = !fold_step(op, acc, arg(C, base, i));
      if (div0) return E_DIV0;
      *out = acc;
      return 0;
    }
    case BI_REM: case BI_MOD: case BI_NUMEQ: case BI_LT: case BI_GT: case BI_LE: case BI_GE:
    case BI_EQ: case BI_EQUAL: case BI_NULL: case BI_NOT: case BI_ATOM: case BI_CONSP:
    case BI_NUMBERP: case BI_SYMBOLP: case BI_CAR: case BI_CDR: case BI_CONS: case BI_LENGTH:
    case BI_REVERSE: case BI_NTH: case BI_SQRT: case BI_FLOAT: case BI_TRUNC: {
      uint32_t need = (op == BI_REM || op == BI_MOD || op == BI_NUMEQ || op == BI_LT || op == BI_GT ||
                       op == BI_LE || op == BI_GE || op == BI_EQ || op == BI_EQUAL || op == BI_CONS ||
                       op == BI_NTH) ? 2 : 1;
      if (cnt != need) return E_ARITY;
      break;
    }
  }
  switch (op) {
    case BI_SQRT: case BI_FLOAT: case BI_TRUNC: {
      V a = arg(C, base, 0);
      if (!is_num(a.t)) return E_TYPE;
      if (op == BI_SQRT) { *out = mkf(__dsqrt_rn(as_f64(a))); return 0; }
      if (op == BI_FLOAT) { *out = mkf(as_f64(a)); return 0; }
      if (a.t == K_INT) { *out = a; return 0; }
      double x = __longlong_as_double((long long)a.w);
      if (isnan(x) || fabs(x) >= 9223372036854775808.0) return E_ARG;
      *out = mkv(K_INT, (uint64_t)__double2ll_rz(x));
      return 0;
    }
    case BI_EQUAL: {
      bool r;
      uint8_t e = equal_values(C, vtop, arg(C, base, 0), arg(C, base, 1), &r);
      if (e) return e;
      *out = mkb(r);
      return 0;
    }
    case BI_CONS: {
      V a = arg(C, base, 0), b = arg(C, base, 1);
      uint32_t c;
      if (!heap_alloc<CHUNK>(H, 3, &c)) return E_OOM;
      uint32_t ca = box_into(H, a, c + 1), cd = box_into(H, b, c + 2);
      H.tag[c] = (uint8_t)(K_CONS | (proper_value(C, b) ? TAG_PROPER : 0));
      H.word[c] = pack2(ca, cd);
      *out = mkv(K_CONS, c);
      return 0;
    }
    case BI_LIST: {
      if (cnt == 0) { *out = mkv(K_NIL, 0); return 0; }
      uint32_t c;
      if (!heap_alloc<CHUNK>(H, 2 * cnt, &c)) return E_OOM;
      for (uint32_t i = 0; i < cnt; ++i) {
        uint32_t ca = box_into(H, arg(C, base, i), c + cnt + i);
        H.tag[c + i] = K_CONS | TAG_PROPER;
        H.word[c + i] = pack2(ca, i + 1 < cnt ? c + i + 1 : 0);
      }
      *out = mkv(K_CONS, c);
      return 0;
    }
    case BI_LENGTH: {
      V a = arg(C, base, 0);
      if (!proper_value(C, a)) return E_TYPE;
      uint64_t n = 0;
      for (uint32_t c = a.t == K_NIL ? 0 : (uint32_t)a.w; c != 0; c = cdr_of(C, c)) ++n;
      *out = mkv(K_INT, n);
      return 0;
    }
    case BI_APPEND: {
      if (cnt == 0) { *out = mkv(K_NIL, 0); return 0; }
      uint32_t total = 0;
      for (uint32_t i = 0; i + 1 < cnt; ++i) {
        V a = arg(C, base, i);
        if (!proper_value(C, a)) return E_TYPE;
        for (uint32_t c = a.t == K_NIL ? 0 : (uint32_t)a.w; c != 0; c = cdr_of(C, c)) ++total;
      }
      V last = arg(C, base, cnt - 1);
      if (total == 0) { *out = last; return 0; }
      uint32_t c;
      if (!heap_alloc<CHUNK>(H, total + 1, &c)) return E_OOM;
      uint32_t tail = box_into(H, last, c + total);
      uint8_t tg = (uint8_t)(K_CONS | (proper_value(C, last) ? TAG_PROPER : 0));
      uint32_t k = 0;
      for (uint32_t i = 0; i + 1 < cnt; ++i) {
        V a = arg(C, base, i);
        for (uint32_t x = a.t == K_NIL ? 0 : (uint32_t)a.w; x != 0;) {
          uint64_t w = nword(C, x);
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
      V a = arg(C, base, 0);
      if (!proper_value(C, a)) return E_TYPE;
      if (a.t == K_NIL) { *out = a; return 0; }
      uint32_t n = 0;
      for (uint32_t x = (uint32_t)a.w; x != 0; x = cdr_of(C, x)) ++n;
      uint32_t c;
      if (!heap_alloc<CHUNK>(H, n, &c)) return E_OOM;
      uint32_t k = 0;
      for (uint32_t x = (uint32_t)a.w; x != 0; ++k) {
        uint64_t w = nword(C, x);
        uint32_t j = n - 1 - k;
        H.tag[c + j] = K_CONS | TAG_PROPER;
        H.word[c + j] = pack2(lo32(w), j + 1 < n ? c + j + 1 : 0);
        x = hi32(w);
      }
      *out = mkv(K_CONS, c);
      return 0;
    }
    case BI_NTH: {
      V i = arg(C, base, 0), l = arg(C, base, 1);
      if (i.t != K_INT || !proper_value(C, l)) return E_TYPE;
      long long k = (long long)i.w;
      if (k < 0) return E_ARG;
      uint32_t x = l.t == K_NIL ? 0 : (uint32_t)l.w;
      for (; k > 0 && x != 0; --k) x = cdr_of(C, x);
      *out = x == 0 ? mkv(K_NIL, 0) : unbox(C, car_of(C, x));
      return 0;
    }
    default: {                                       // fast ops with arity errors (cnt > 2)
      V a0 = arg(C, base, 0), a1 = arg(C, base, 1);
      return fast2_full(C, op, cnt > 2 ? 3 : cnt, a0, a1, out);
    }
  }
}

// (||| n f l1 .. lm) argument checks (c.7): arity, types left to right, then n >= 0 and every list
// proper with >= n elements.  Returns 0 and fills n, or an error.
__device__ CULI_COLD uint8_t par_check(Ctx C, uint32_t base, uint32_t cnt, uint32_t* n_out) {
  if (cnt < 3) return E_ARITY;
  V nv = arg(C, base, 0), f = arg(C, base, 1);
  if (nv.t != K_INT) return E_TYPE;
  if (f.t != K_BUILTIN && f.t != K_CLOSURE) return E_TYPE;
  long long n = (long long)nv.w;
  if (n < 0) return E_ARG;
  for (uint32_t j = 2; j < cnt; ++j) {
    V l = arg(C, base, j);
    if (!proper_value(C, l)) return E_ARG;
    uint32_t c = l.t == K_NIL ? 0 : (uint32_t)l.w;
    long long q = 0;
    for (; q < n && c != 0; ++q) c = cdr_of(C, c);
    if (q < n) return E_ARG;
  }
  if (n > 0x3fffffffll) return E_OOM;
  *n_out = (uint32_t)n;
  return 0;
}

// The O(1) part of par_check: arity, types, n >= 0, every list proper, and no empty list when n > 0.
__device__ CULI_COLD uint8_t par_check_light(Ctx C, uint32_t base, uint32_t cnt, uint32_t* n_out) {
  if (cnt < 3) return E_ARITY;
  V nv = arg(C, base, 0), f = arg(C, base, 1);
  if (nv.t != K_INT) return E_TYPE;
  if (f.t != K_BUILTIN && f.t != K_CLOSURE) return E_TYPE;
  long long n = (long long)nv.w;
  if (n < 0) return E_ARG;
  for (uint32_t j = 2; j < cnt; ++j) {
    V l = arg(C, base, j);
    if (!proper_value(C, l)) return E_ARG;
    if (n > 0 && l.t == K_NIL) return E_ARG;
  }
  if (n > 0x3fffffffll) return E_OOM;
  *n_out = (uint32_t)n;
  return 0;
}

// runtime syntax checks of special forms without TAG_VALID (c.5); cur = the argument list
__device__ CULI_COLD bool special_syntax_ok(Ctx C, uint32_t op, uint32_t cur) {
  uint32_t n = 0;
  for (uint32_t c = cur; c != 0; c = cdr_of(C, c)) ++n;
  switch (op) {
    case SP_QUOTE: return n == 1;
    case SP_IF: return n == 2 || n == 3;
    case SP_PROGN: return true;
    case SP_LAMBDA: return n >= 1 && valid_params(C, car_of(C, cur));
    case SP_DEFINE:
    case SP_SETQ: return n == 2 && bindable_node(C, car_of(C, cur));
    case SP_DEFUN: case SP_DEFMACRO:
      return n >= 2 && bindable_node(C, car_of(C, cur)) && valid_params(C, car_of(C, cdr_of(C, cur)));
    case SP_QUASIQUOTE: return n == 1;
    case SP_LET: {
      if (n < 1) return false;
      uint32_t bl = car_of(C, cur);
      if (bl != 0) {
        uint32_t bt = ntag(C, bl);
        if ((bt & KIND_MASK) != K_CONS || !(bt & TAG_PROPER)) return false;
        for (uint32_t c = bl; c != 0; c = cdr_of(C, c)) {
          uint32_t b = car_of(C, c);
          uint32_t tb = ntag(C, b);
          if ((tb & KIND_MASK) != K_CONS || !(tb & TAG_PROPER)) return false;
          uint64_t bw = nword(C, b);
          if (!bindable_node(C, lo32(bw))) return false;
          uint32_t r = hi32(bw);
          if (r == 0 || cdr_of(C, r) != 0) return false;
        }
      }
      return true;
    }
  }
  return false;
}

// ---- leaf forms ------------------------------------------------------------------------------------------
// x (tag xt, word xw) is a list whose own eval step was already counted at depth dx.  If x is a *leaf*
// (op a [b]) — op a reserved builtin of FAST_OPS, a and b atoms or symbols — evaluate it right here:
// the head step, then each argument step (all at depth dx + 1, with the fuel/depth checks in the same
// order as the recursive definition, c.4), then the builtin.  Returns 1 with *out, 2 with *err, or 0
// (not a leaf: nothing counted, nothing changed).  Saves the continuation push/pop of the common
// arithmetic leaves, e.g. (- n 1), (< n 2), (* k x).
__device__ __forceinline__ int try_leaf(const Ctx& C, uint32_t xt, uint64_t xw, uint32_t dx, uint32_t env,
                                        uint64_t& steps, uint64_t fuel, uint32_t maxd, V* out, uint8_t* err) {
  if (!(xt & TAG_PROPER)) return 0;
  // round 1 (independent loads): the head node, the first argument cell and — speculatively, since
  // reader spines are contiguous (c.14) — the cell after it
  uint32_t c1 = hi32(xw);
  uint32_t ht;
  uint64_t hw;
  ldnode(C, lo32(xw), ht, hw);
  uint64_t cw1 = C.A->H.word[c1];                     // c1 == 0 reads the nil node: harmless
  uint64_t cw2s = C.A->H.word[c1 + 1 < C.A->H.cap ? c1 + 1 : 0];
  if ((ht & KIND_MASK) != K_SYM || hw < N_SPECIALS || hw >= N_RESERVED) return 0;
  uint32_t op = (uint32_t)hw - N_SPECIALS;
  if (!((FAST_OPS >> op) & 1)) return 0;
  uint32_t argc = 0, n1 = 0, n2 = 0, t1 = 0, t2 = 0;
  uint64_t w1 = 0, w2 = 0;
  if (c1 != 0) {
    n1 = lo32(cw1);
    uint32_t c2 = hi32(cw1);
    uint64_t cw2 = c2 == c1 + 1 ? cw2s : C.A->H.word[c2];
    // round 2: both argument nodes
    ldnode(C, n1, t1, w1);
    if (c2 != 0) ldnode(C, lo32(cw2), t2, w2);
    if ((t1 & KIND_MASK) == K_CONS) return 0;
    argc = 1;
    if (c2 != 0) {
      if (hi32(cw2) != 0) return 0;
      n2 = lo32(cw2);
      if ((t2 & KIND_MASK) == K_CONS) return 0;
      argc = 2;
    }
  }
  // head step, then one step per argument (argc + 1 steps at depth dx + 1), checked at once; on failure
  // the first failing step decides: fuel before depth at each step (c.4 step 1)
  if (__builtin_expect(steps + argc + 1 > fuel || dx + 1 > maxd, 0)) {
    if (steps + 1 > fuel || dx + 1 <= maxd) {
      *err = E_FUEL;
      steps = fuel + 1;
    } else {
      *err = E_DEPTH;
      steps = steps + 1;
    }
    return 2;
  }
  steps += argc + 1;
  V a0 = mkv(K_NIL, 0), a1 = mkv(K_NIL, 0);
  if (argc > 0) a0 = (t1 & KIND_MASK) == K_SYM ? lookup(C, (uint32_t)w1, env) : unbox_loaded(n1, t1, w1);
  if (argc > 1) a1 = (t2 & KIND_MASK) == K_SYM ? lookup(C, (uint32_t)w2, env) : unbox_loaded(n2, t2, w2);
  uint8_t e = fast2(C, op, argc, a0, a1, out);
  if (__builtin_expect(e != 0, 0)) { *err = e; return 2; }
  return 1;
}

// ---- quasiquote (reading R8) ----------------------------------------------------
// The quasiquote operator a template list starts with (its head node), else 0xff.
__device__ __forceinline__ uint32_t qq_op(const Ctx& C, uint64_t listword) {
  uint32_t ht;
  uint64_t hw;
  ldnode(C, lo32(listword), ht, hw);
  if ((ht & KIND_MASK) != K_SYM) return 0xffu;
  return (hw == SP_QUASIQUOTE || hw == SP_UNQUOTE || hw == SP_UNQUOTE_SPLICING) ? (uint32_t)hw : 0xffu;
}
// The single argument of a proper (op x) whose cell word is `listword`; false: not exactly one argument.
__device__ __forceinline__ bool qq_arg(const Ctx& C, uint64_t listword, uint32_t* arg) {
  uint32_t rest = hi32(listword);
  if (rest == 0) return false;
  uint64_t rw = nword(C, rest);
  if (hi32(rw) != 0) return false;
  *arg = lo32(rw);
  return true;
}

// try_leaf out of line (CULI_LEAF_CALL=1): one copy of the leaf evaluator (and of the symbol lookups it
// inlines) instead of four — the machine is instruction-fetch bound, at the price of a call.
#ifndef CULI_LEAF_CALL
#define CULI_LEAF_CALL 0
#endif
struct LeafOut {
  V v;
  uint64_t steps;
  int kind;
  uint8_t err;
};
__device__ __noinline__ LeafOut try_leaf_call(Ctx C, uint32_t xt, uint64_t xw, uint32_t dx, uint32_t env,
                                              uint64_t steps, uint64_t fuel, uint32_t maxd) {
  LeafOut o;
  o.steps = steps;
  o.err = 0;
  o.v = mkv(K_NIL, 0);
  o.kind = try_leaf(C, xt, xw, dx, env, o.steps, fuel, maxd, &o.v, &o.err);
  return o;
}
#if CULI_LEAF_CALL
#define TRY_LEAF(res, outv)                                                               \
  do {                                                                                    \
    LeafOut lo_ = try_leaf_call(C, at, aw, d + 1, env, steps, fuel, maxd);                \
    res = lo_.kind;                                                                       \
    steps = lo_.steps;                                                                    \
    if (res == 1) outv = lo_.v; else if (res == 2) err = lo_.err;                         \
  } while (0)
#else
#define TRY_LEAF(res, outv) res = try_leaf(C, at, aw, d + 1, env, steps, fuel, maxd, &outv, &err)
#endif

// ---- the machine ---------------------------------------------------------------------------------------
enum KKind : uint32_t { KF_HEAD = 1, KF_ARGS, KF_BODY, KF_IF, KF_LET, KF_DEFINE, KF_MACRO, KF_PAR, KF_DATA, KF_QQ,
                       KF_JOIN, KF_SETQ };   // KF_JOIN: a KF_ARGS frame whose next argument was split off

// ---- argument splitting ----------------------------------------------------------------
__device__ __forceinline__ uint32_t ld_acquire(const uint32_t* p) {
  uint32_t v;
  asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_release(uint32_t* p, uint32_t v) {
  asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

__device__ __forceinline__ unsigned long long gtime() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}
__device__ __forceinline__ unsigned long long ld_acquire64(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ unsigned long long ld_relaxed64(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}

// Warp-aggregated fetch-and-add of 1 per calling lane (the lanes executing it together share one atomic
// and get consecutive values in lane order).  Safe in diverged code: the mask is the lanes present, and no
// other collective can run between __activemask and the shuffle (the leader's branch holds only the atomic).
__device__ __forceinline__ unsigned long long fetch_add_lanes(unsigned long long* p) {
  unsigned mask = __activemask();
  int lane = threadIdx.x & 31;
  int leader = __ffs(mask) - 1;
  unsigned rank = __popc(mask & ((1u << lane) - 1u));
  unsigned long long base = 0;
  if (lane == leader) base = atomicAdd(p, (unsigned long long)__popc(mask));
  base = __shfl_sync(mask, base, leader);
  return base + rank;
}
__device__ __forceinline__ uint32_t fetch_add_lanes32(uint32_t* p) {
  unsigned mask = __activemask();
  int lane = threadIdx.x & 31;
  int leader = __ffs(mask) - 1;
  unsigned rank = __popc(mask & ((1u << lane) - 1u));
  uint32_t base = 0;
  if (lane == leader) base = atomicAdd(p, (uint32_t)__popc(mask));
  base = __shfl_sync(mask, base, leader);
  return base + rank;
}

// fetch_add_lanes32 for lanes that may address different counters: the lanes executing it together are
// grouped by address (__match_any_sync, restricted to the caller's mask), one atomic per group.
__device__ __forceinline__ uint32_t fetch_add_grouped(uint32_t* p) {
  unsigned mask = __activemask();
  unsigned peers = __match_any_sync(mask, (unsigned long long)p) & mask;
  int lane = threadIdx.x & 31;
  int leader = __ffs(peers) - 1;
  unsigned rank = __popc(peers & ((1u << lane) - 1u));
  uint32_t base = 0;
  if (lane == leader) base = atomicAdd(p, (uint32_t)__popc(peers));
  base = __shfl_sync(peers, base, leader);
  return base + rank;
}

// A bounded wait gave up: count it and keep the first occurrence's state for diagnosis.
// Every wait on another lane is bounded by EvalArgs.wait_ns, so a protocol bug shows up as a counter and a
// status (culi_last_waits), never as a frozen GPU.
__device__ CULI_COLD void wait_gave_up(const EvalArgs& A, uint32_t kind, uint32_t g, uint32_t form) {
  if (atomicAdd(&A.sctl->timeouts, 1u) != 0) return;
  uint32_t* d = A.sctl->diag;
  d[0] = kind;
  d[1] = g;
  d[2] = threadIdx.x & 31;
  d[3] = form;
  if (kind == WAIT_JOIN) {
    const SplitGroup* G = A.groups + g;
    d[4] = *(volatile const uint32_t*)&G->state;
    d[5] = *(volatile const uint32_t*)&G->mask;
    d[6] = *(volatile const uint32_t*)&G->remaining;
    d[7] = *(volatile const uint32_t*)&G->t[threadIdx.x & 31].done;
    d[8] = *(volatile const uint32_t*)&G->claimer;
  }
  __threadfence();
}

#if CULI_WATCHDOG
__device__ CULI_COLD bool watchdog_fired(Ctx C, uint32_t form, uint64_t steps, uint32_t sp, uint32_t d, uint32_t root) {
  const EvalArgs& A = *C.A;
  if (gtime() - *(volatile unsigned long long*)&A.sctl->t0 < (unsigned long long)CULI_WATCHDOG * 1000000ull) return false;
  if (atomicAdd(&A.sctl->wd[0], 1u) == 0) {
    uint32_t* w = A.sctl->wd;
    w[1] = form; w[2] = (uint32_t)steps; w[3] = sp; w[4] = d; w[5] = root; w[6] = 0;
    w[7] = *(volatile uint32_t*)A.finished;
  }
  return true;
}
#endif

// In-use bits of the SPLIT_GPW group slots of each warp of the block (the block has 4 warps); cleared by
// the kernel prologue, set by try_split (atomic test-and-set), cleared by the last owner lane that joins.
__shared__ uint32_t culi_split_busy[4];

__device__ __forceinline__ uint32_t my_slot() { return blockIdx.x * blockDim.x + threadIdx.x; }

// Called by a lane at a poll point (its top continuation already flushed to memory).  If an idle warp waits
// for work (head > tail), each polling lane looks for the outermost KF_ARGS frame whose next argument is an
// unevaluated list and copies that frame's environment to the heap (promote).  Then the lanes that poll
// together (__activemask(): typically a converged warp of same-shaped forms) publish their arguments as one
// group: the first lane takes a free group slot of the warp, each lane with an argument writes task `lane`
// and turns its frame into KF_JOIN (the V-stack header records the group), and the group goes into the
// queue with one ticket.  Each owner lane later joins (RET KF_JOIN); the first to find the group unclaimed
// takes the whole group back.
// (Warp intrinsics only as __activemask -> ballot/shuffle over that mask with no other collective in
// between, results restricted to the mask: a lane group of the same warp inside its own call can execute
// the same instruction converged with ours.  DESIGN.md §5.5.)
__device__ CULI_COLD void try_split(Ctx C, uint32_t sp, uint64_t steps, uint64_t fuel, uint32_t form) {
  const EvalArgs& A = *C.A;
  SplitCtl* Q = A.sctl;
  uint32_t* busy = &culi_split_busy[threadIdx.x >> 5];
  bool have = false;
  uint32_t lvl = 0xffffffffu, henv = 0;
  uint4 fr = make_uint4(0, 0, 0, 0);
  unsigned long long tail = ld_relaxed64(&Q->tail), head = ld_relaxed64(&Q->head);
  if (head > tail && (~*(volatile uint32_t*)busy & ((1u << SPLIT_GPW) - 1u))) {
    for (uint32_t i = 0; i < sp; ++i) {
      uint4 f = *KS(C, i);
      if (kkind(f.w) == KF_ARGS && f.x != 0 && (ntag(C, car_of(C, f.x)) & KIND_MASK) == K_CONS) {
        lvl = i;
        fr = f;
        break;
      }
    }
    have = lvl != 0xffffffffu && promote(C, fr.y, &henv);
  }
  unsigned m = __activemask();
  unsigned part = __ballot_sync(m, have) & m;
  if (!part) return;
  int lane = threadIdx.x & 31, leader = __ffs(part) - 1;
  int j = -1;
  if (lane == leader) {                                         // one atomic test-and-set of a free slot
    // (no retry loop: a spinning leader between two collectives let the other lanes pass the shuffle
    // without it on sm_100a, a deadlock; a lost race just skips this poll)
    uint32_t freeb = ~*(volatile uint32_t*)busy & ((1u << SPLIT_GPW) - 1u);
    uint32_t bit = freeb & (0u - freeb);
    if (bit && !(atomicOr(busy, bit) & bit)) j = __ffs(bit) - 1;
  }
  j = __shfl_sync(m, j, leader);
  if (j < 0) return;                                            // (promoted frames stay valid copies)
  uint32_t g = my_slot() / 32 * SPLIT_GPW + (uint32_t)j;
  SplitGroup* G = A.groups + g;
  if (have) {
    SplitTask* T = &G->t[lane];
    T->expr = car_of(C, fr.x);
    T->env = henv;
    T->depth = kdepth(fr.w) + 1;                                // arguments run at depth d + 1
    T->budget = fuel - steps;
    T->done = 0;
    KS(C, lvl)->w = (fr.w & ~(0xfu << 12)) | (KF_JOIN << 12);
    VS(C, fr.z)->z = g + 1;                                     // the call's header: the group
  }
  // every task written: bar.warp.sync orders the lanes' writes before the leader's release below (no
  // fence.sc: it would invalidate the SM's L1)
  __syncwarp(m);
  if (lane == leader) {
    G->mask = part;
    G->remaining = __popc(part);
    G->form = form;
    G->claimer = 0xffffffffu;
    st_release(&G->state, SPLIT_OPEN);
    unsigned long long q = atomicAdd(&Q->tail, 1ull);
    atomicAdd(&Q->published, 1u);
    unsigned long long e = ((q & 0xffffffffull) << 32) | (g + 1);
    asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(&A.gqueue[q & (A.gqcap - 1)]), "l"(e) : "memory");
  }
}

// the owner lane is done with group g: the last one frees the warp's slot
__device__ __forceinline__ void group_release(const EvalArgs& A, uint32_t g) {
  if (atomicSub(&A.groups[g].remaining, 1u) == 1u)
    atomicAnd(&culi_split_busy[threadIdx.x >> 5], ~(1u << (g % SPLIT_GPW)));
}

// Owner side of a join whose group a thief claimed: wait for this lane's task (bounded).  false = the wait
// gave up; the owner then evaluates the argument itself and does not release the group, so its slot stays
// busy for the rest of the launch and a late thief can never write into a reused group.
// The poll is a relaxed load: an acquire (ld.acquire / fence.sc) invalidates the SM's whole L1 on sm_100a
// (CCTL.IVALL), and waiting owners polling every 200 ns did so 490 M times per C2 launch, evicting the
// stacks and code of every busy warp on the SM (ncu).  One acquire once the flag is seen.
__device__ __forceinline__ uint32_t ld_relaxed(const uint32_t* p) {
  uint32_t v;
  asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ CULI_COLD bool join_wait(const EvalArgs& A, SplitTask* T, uint32_t g, uint32_t form) {
  unsigned long long t0 = gtime();
  uint32_t ns = 128;
  for (uint32_t spin = 1;; ++spin) {
    if (ld_relaxed(&T->done) != 0) {
      ld_acquire(&T->done);
      return true;
    }
    __nanosleep(ns);
    ns = ns < A.split_sleep ? ns * 2 : ns;                      // (polling warps cost issue slots and I$)
    if ((spin & 15) == 0 && gtime() - t0 > A.wait_ns) {
      wait_gave_up(A, WAIT_JOIN, g, form);
      return false;
    }
  }
}

// A lane leaves its evaluation with an error while KF_JOIN frames are on its stack: hand their groups back
// (still open: take the group back and release this lane's share); a claimed group stays busy until the
// launch ends (its thief still writes it).
__device__ CULI_COLD void abandon_joins(Ctx C, uint32_t sp, uint4 ktop) {
  const EvalArgs& A = *C.A;
  for (uint32_t i = 0; i < sp; ++i) {
    uint4 f = i + 1 == sp ? ktop : *KS(C, i);
    if (kkind(f.w) != KF_JOIN) continue;
    uint32_t g = VS(C, f.z)->z - 1;
    uint32_t st = atomicCAS(&A.groups[g].state, SPLIT_OPEN, SPLIT_TAKEN);
    if (st == SPLIT_OPEN || st == SPLIT_TAKEN) group_release(A, g);
  }
}

struct FormOut {
  uint32_t t;
  uint64_t w;
  uint64_t steps;
  uint8_t err;
  uint32_t aux;        // E_SUSPEND: index of the nested-||| descriptor; E_YIELD: stack height
  uint32_t vtop;       // E_YIELD: V-stack top
  uint32_t kk;         // E_YIELD: kind of the continuation about to be popped
};

// state to resume a suspended evaluation at RET with value v (the nested |||'s result, or the value a
// yielding lane was about to return); grp / wait: VOTE mode, see eval_form
struct Resume {
  uint32_t sp, vtop;
  uint64_t steps;
  V v;
  uint32_t grp, wait;
};

// eval_form(C, root, form, 0, 0, fuel): evaluate the datum at node `root` at depth 1.
// eval_form(C, 0, form, 1, m, budget): apply vs[0] to the m values vs[1..m] as the body of a top-level
//   (||| ...) form (depth 1) — one fan-out element (c.7); `budget` = fuel left after the ||| arguments.
// eval_form<..., SPLIT>(C, root, form, 0, 0, budget, depth, false, {}, env): a split-off argument task.
// VOTE: the lanes of R.grp run together; at a return, a lane yields (E_YIELD, state in FormOut) when its
// group is no longer converged (__activemask() != grp) or its stack is back down to the height R.wait of
// the deepest waiting lane, where the two groups can continue as one.
template <bool FANOUT, bool APPLY, bool NEST = false, bool SPLIT = false, bool VOTE = false>
__device__ __forceinline__ FormOut eval_form(const Ctx& C, uint32_t root, uint32_t form, int apply_mode,
                                             uint32_t apply_cnt, uint64_t fuel, uint32_t d0 = 1,
                                             bool resume = false, const Resume& R = Resume{},
                                             uint32_t env0 = 0) {
  const DevHeap& H = C.A->H;
  const uint32_t kcap = C.A->kcap, vcap = C.A->vcap, maxd = C.A->max_depth;
  const bool fanout = FANOUT && !APPLY && C.A->fanout;
  V v = mkv(K_NIL, 0), a0 = mkv(K_NIL, 0), a1 = mkv(K_NIL, 0);
  uint32_t x = root, t = 0, env = env0, d = d0, cur = 0, base = 0, cnt = 0, sp = 0, vtop = 0;
  uint32_t a = 0, at = 0, nxt = 0, kd = 0, hop = 0, qlev = 0;
  uint64_t w = 0, aw = 0, w0 = 0;
  uint64_t steps = 0;
  uint8_t err = 0;
  uint4 k, ktop = make_uint4(0, 0, 0, 0);
  uint4 hv = make_uint4(0, 0, 0, 0);      // the value being applied (copy of vs[base])
  bool kdirty = false;                      // ktop holds frame sp-1 not yet written to memory
  uint32_t pollc = SPLIT ? C.A->split_first : 0;  // closure calls until the next split poll

#define FAIL(e) do { err = (e); goto done; } while (0)
// setq batches (R7): a frame moves to the heap as soon as it is made, so that no copy of it can go stale
#define MUT_FRAME() do { uint32_t h_; if (__builtin_expect(!!(!promote(C, env, &h_)), 0)) FAIL(E_OOM); env = h_; } while (0)
#if CULI_WATCHDOG
#define WATCHDOG() do { if ((steps & 0x3fff) == 0 && watchdog_fired(C, form, steps, sp, d, root)) FAIL(E_OOM); } while (0)
#else
#define WATCHDOG() do { } while (0)
#endif
#define STEP(depth)                                     \
  do {                                                  \
    ++steps;                                            \
    WATCHDOG();                                         \
    if (__builtin_expect(steps > fuel || (depth) > maxd, 0)) { \
      err = steps > fuel ? E_FUEL : E_DEPTH;            \
      goto done;                                        \
    }                                                   \
  } while (0)
#define KPUSH(kind, cursor, envv, vsb, depth, count)                                  \
  do {                                                                                \
    if (__builtin_expect(!!(sp >= kcap), 0)) FAIL(E_OOM);                                                      \
    if (kdirty) *KS(C, sp - 1) = ktop;                                                \
    ktop = make_uint4((cursor), (envv), (vsb), kmeta((depth), (kind), (count)));      \
    kdirty = true;                                                                    \
    ++sp;                                                                             \
  } while (0)
#define ATOMVAL(n, tt, ww) (((tt) & KIND_MASK) == K_SYM ? lookup(C, (uint32_t)(ww), env) : unbox_loaded((n), (tt), (ww)))

  uint32_t aux = 0;
  if ((NEST || VOTE) && resume) {                               // continue a suspended evaluation
    sp = R.sp;
    vtop = R.vtop;
    steps = R.steps;
    v = R.v;
    if (sp > 0) ktop = *KS(C, sp - 1);
    goto RET_POP;                                               // (no yield check: make progress first)
  }
  if (APPLY && apply_mode) {
    base = 0;
    hv = *VS(C, 0);
    cnt = apply_cnt;
    vtop = 1 + cnt;
    goto APPLY;
  }
  // ======================================================== EVAL a code node x in env at depth d
EVAL_NODE:
  ldnode(C, x, t, w);
EVAL_NODE_LOADED:
  STEP(d);                                                      // one canonical step (c.4 step 1)
  if ((t & KIND_MASK) != K_CONS) { v = ATOMVAL(x, t, w); goto RET; }   // symbol / self-evaluating
  // ======================================================== a list x (its step already counted)
EVAL_CONS:
  if (__builtin_expect(!(t & TAG_PROPER), 0)) FAIL(E_SYNTAX);
  a = lo32(w);
  cur = hi32(w);
  ldnode(C, a, at, aw);
  STEP(d + 1);                                                  // the head is always evaluated first
  if ((at & KIND_MASK) != K_CONS) { v = ATOMVAL(a, at, aw); goto HEAD; }   // (L440-441)
  KPUSH(KF_HEAD, cur, env, vtop, d, 0);
  x = a; t = at; w = aw; d = d + 1;
  goto EVAL_CONS;

  // ======================================================== EVAL a value (a macro expansion)
EVAL_VALUE:
  STEP(d);
  if (v.t == K_SYM) { v = lookup(C, (uint32_t)v.w, env); goto RET; }
  if (v.t != K_CONS) goto RET;
  x = (uint32_t)v.w;
  ldnode(C, x, t, w);
  goto EVAL_CONS;

  // ======================================================== head value v, unevaluated args `cur`
HEAD:
  if (FANOUT && !APPLY && fanout && sp == 0 && d == 1 && C.A->wide && C.A->wide[form] >= WIDE_MIN) {
    // a wide top-level form (K12): evaluate its arguments one per thread in the fan-out kernel
    uint32_t kind = 0xffu, op = 0;
    if (v.t == K_BUILTIN && v.w == BI_LIST) kind = FAN_LIST;
    else if (v.t == K_BUILTIN && (v.w == BI_ADD || v.w == BI_MUL)) { kind = FAN_FOLD; op = (uint32_t)v.w; }
    else if (v.t != K_BUILTIN && v.t != K_SPECIAL && v.t != K_CLOSURE && v.t != K_MACRO) kind = FAN_DATA;
    if (kind != 0xffu) {
      uint32_t slot = atomicAdd(C.A->npend, 1u);
      if (slot < C.A->maxdesc) {
        uint32_t nargs = C.A->wide[form];
        uint32_t ncells = kind == FAN_DATA ? nargs + 1 : nargs, spine;
        if (__builtin_expect(!!(!heap_alloc<!VOTE>(H, kind == FAN_FOLD ? nargs : 2 * ncells, &spine)), 0)) FAIL(E_OOM);
        if (kind == FAN_DATA) {                                   // cell 0 holds the head value
          uint32_t ca = box_into(H, v, spine + ncells);
          H.tag[spine] = K_CONS | TAG_PROPER;
          H.word[spine] = pack2(ca, ncells > 1 ? spine + 1 : 0);
        }
        FanDesc* D = C.A->desc + slot;
        D->form = form;
        D->n = ncells;
        D->m = op;
        D->kind = kind;
        D->nelem = nargs;
        D->spine = spine;
        D->ftag = v.t;
        D->depth = d;
        D->fword = v.w;
        D->steps0 = steps;
        D->top = atomicAdd(H.top, 0ull);
        D->heads[0] = cur;
        D->total = 0;
        D->bad = 0;
        D->nonflat = 0;
        err = E_PENDING;
        goto done;
      }
    }
  }
  if (v.t == K_BUILTIN && ((FAST_OPS >> v.w) & 1)) {            // register fast path
    hop = (uint32_t)v.w;
    cnt = 0;
    while (cur != 0) {
      w0 = nword(C, cur);
      a = lo32(w0);
      nxt = hi32(w0);
      ldnode(C, a, at, aw);
      STEP(d + 1);
      int leaf = 0;
      V av;
      if ((at & KIND_MASK) == K_CONS) {
        TRY_LEAF(leaf, av);
        if (__builtin_expect(leaf == 2, 0)) goto done;
      } else {
        av = ATOMVAL(a, at, aw);
      }
      if ((at & KIND_MASK) == K_CONS && leaf == 0 || cnt == 2) {   // spill to the general path
        if (__builtin_expect(!!(vtop + 3 >= vcap), 0)) FAIL(E_OOM);
        base = vtop;
        hv = vpack(mkv(K_BUILTIN, hop), 0);
        *VS(C, base) = hv;
        if (cnt > 0) *VS(C, base + 1) = vpack(a0, 0);
        if (cnt > 1) *VS(C, base + 2) = vpack(a1, 0);
        if ((at & KIND_MASK) == K_CONS && leaf == 0) {
          vtop = base + 1 + cnt;
          KPUSH(KF_ARGS, nxt, env, base, d, cnt);
          x = a; t = at; w = aw; d = d + 1;
          goto EVAL_CONS;
        }
        *VS(C, base + 1 + cnt) = vpack(av, 0);
        ++cnt;
        cur = nxt;
        goto ARGS;
      }
      if (cnt == 0) a0 = av; else a1 = av;
      ++cnt;
      cur = nxt;
    }
    {
      uint8_t e = fast2(C, hop, cnt, a0, a1, &v);
      if (__builtin_expect(!!(e), 0)) FAIL(e);
    }
    goto RET;
  }
  if (v.t == K_SPECIAL) {
    uint32_t op = (uint32_t)v.w;
    if (op == SP_DEFINE || op == SP_DEFUN || op == SP_DEFMACRO) {
      if (__builtin_expect(!!(!C.A->define_mode), 0)) FAIL(E_DEFINE_IN_BATCH);
    }
    if (__builtin_expect(!!(!(t & TAG_VALID) && !special_syntax_ok(C, op, cur)), 0)) FAIL(E_SYNTAX);
    if (__builtin_expect(op >= SP_QUASIQUOTE, 0)) goto QQ_SPECIAL;   // R8 (cold code below)
    switch (op) {
      case SP_IF: {
        w0 = nword(C, cur);
        uint32_t c1 = hi32(w0);
        a = lo32(w0);
        ldnode(C, a, at, aw);
        STEP(d + 1);
        if ((at & KIND_MASK) == K_CONS) {
          int leaf;
          TRY_LEAF(leaf, v);
          if (__builtin_expect(leaf == 2, 0)) goto done;
          if (leaf == 0) {
            KPUSH(KF_IF, c1, env, vtop, d, 0);
            x = a; t = at; w = aw; d = d + 1;
            goto EVAL_CONS;
          }
        } else {
          v = ATOMVAL(a, at, aw);
        }
        cur = c1;
        goto IF_BRANCH;
      }
      case SP_QUOTE:
        v = unbox(C, car_of(C, cur));
        goto RET;
      case SP_PROGN:
        goto BODY;
      case SP_LAMBDA:
        if (__builtin_expect(!!(!make_closure(C, K_CLOSURE, cur, env, &v)), 0)) FAIL(E_OOM);
        goto RET;
      case SP_LET: {
        w0 = nword(C, cur);
        uint32_t bl = lo32(w0), body = hi32(w0);
        if (bl == 0) { cur = body; goto BODY; }
        if (__builtin_expect(!!(vtop >= vcap), 0)) FAIL(E_OOM);
        base = vtop;
        *VS(C, base) = make_uint4(body, 0, 0, K_FRAME);         // header (holds the body for now)
        cnt = 0;
        cur = bl;
        goto LET_LOOP;
      }
      case SP_SETQ: {                                           // R7: the value first, then the binding
        w0 = nword(C, cur);
        KPUSH(KF_SETQ, (uint32_t)nword(C, lo32(w0)), env, vtop, d, 0);
        x = car_of(C, hi32(w0));
        d = d + 1;
        goto EVAL_NODE;
      }
      case SP_DEFINE: {
        w0 = nword(C, cur);
        KPUSH(KF_DEFINE, (uint32_t)nword(C, lo32(w0)), env, vtop, d, 0);
        x = car_of(C, hi32(w0));
        d = d + 1;
        goto EVAL_NODE;
      }
      default: {                                                // defun / defmacro
        w0 = nword(C, cur);
        uint32_t s = (uint32_t)nword(C, lo32(w0));
        V clo;
        if (__builtin_expect(!!(!make_closure(C, op == SP_DEFUN ? K_CLOSURE : K_MACRO, hi32(w0), env, &clo)), 0)) FAIL(E_OOM);
        H.gtag[s] = (uint8_t)clo.t;
        H.gword[s] = clo.w;
        v = mkv(K_SYM, s);
        goto RET;
      }
    }
  }
  if (__builtin_expect(v.t == K_MACRO, 0)) goto MACRO_CALL;    // c.4 MACRO branch (code below RET)
  // data list (L443-444) or (list ...): elements stream into a preallocated contiguous spine (c.14)
  if ((v.t != K_BUILTIN && v.t != K_CLOSURE) || (v.t == K_BUILTIN && v.w == BI_LIST)) goto DATA_START;
  // BUILTIN or CLOSURE: evaluate the args left to right at depth d+1 onto the V-stack
  if (__builtin_expect(!!(vtop >= vcap), 0)) FAIL(E_OOM);
  base = vtop;
  hv = vpack(v, 0);
  *VS(C, base) = hv;
  cnt = 0;
  // fallthrough
ARGS:
  while (cur != 0) {
    w0 = nword(C, cur);
    a = lo32(w0);
    nxt = hi32(w0);
    ldnode(C, a, at, aw);
    STEP(d + 1);
    V av;
    if ((at & KIND_MASK) == K_CONS) {
      int leaf;
      TRY_LEAF(leaf, av);
      if (__builtin_expect(leaf == 2, 0)) goto done;
      if (leaf == 0) {
        vtop = base + 1 + cnt;
        KPUSH(KF_ARGS, nxt, env, base, d, cnt);
        x = a; t = at; w = aw; d = d + 1;
        goto EVAL_CONS;
      }
    } else {
      av = ATOMVAL(a, at, aw);
    }
    if (__builtin_expect(!!(base + 1 + cnt >= vcap), 0)) FAIL(E_OOM);
    *VS(C, base + 1 + cnt) = vpack(av, 0);
    ++cnt;
    cur = nxt;
  }
  vtop = base + 1 + cnt;
  // fallthrough
APPLY: {                                                        // apply vs[base] to cnt args
  V h = vunpack(hv);
  if (h.t == K_CLOSURE) {                                       // PAPER L456-460, c.4 CLOSURE
    if (SPLIT && __builtin_expect(--pollc == 0, 0)) {
      pollc = C.A->split_poll;
      // (the common answer — no idle warp waits for a ticket — without the call and its register traffic)
      if (ld_relaxed64(&C.A->sctl->head) > ld_relaxed64(&C.A->sctl->tail)) {
        if (kdirty) *KS(C, sp - 1) = ktop;
        kdirty = false;
        try_split(C, sp, steps, fuel, form);
        if (sp > 0) ktop = *KS(C, sp - 1);                      // the top frame may have become KF_JOIN
      }
    }
    uint64_t cwd = nword(C, (uint32_t)h.w);                     // three independent loads
    uint64_t aux = nword(C, (uint32_t)h.w + 1);
    uint64_t aux2 = nword(C, (uint32_t)h.w + 2);
    uint32_t np = lo32(aux);
    if (__builtin_expect(!!(np != cnt), 0)) FAIL(E_ARITY);
    uint32_t body = lo32(aux2);
    if (np == 1) {
      VS(C, base + 1)->z = hi32(aux);
    } else {
      uint32_t ps = hi32(aux2);
      for (uint32_t i = 0; i < cnt; ++i) {
        uint64_t pw = nword(C, ps);
        VS(C, base + 1 + i)->z = (uint32_t)nword(C, lo32(pw));
        ps = hi32(pw);
      }
    }
    if (__builtin_expect(!!(cnt >= 0x8000u), 0)) FAIL(E_OOM);
    *VS(C, base) = make_uint4(hi32(cwd), 0, cnt, K_FRAME);
    env = stack_env(base, cnt);
    if (C.A->mut) MUT_FRAME();
    vtop = base + 1 + cnt;
    cur = body;
    goto BODY;
  }
  if (__builtin_expect(!!(h.t != K_BUILTIN), 0)) FAIL(E_SYNTAX);
  if ((uint32_t)h.w == BI_PAR) goto PAR_APPLY;                 // (||| n f l1 ... lm), c.7 (below RET)
  {
    uint8_t e = apply_builtin<!VOTE>(C, (uint32_t)h.w, base, cnt, vtop, &v);
    if (__builtin_expect(!!(e), 0)) FAIL(e);
  }
  vtop = base;
  goto RET;
}

  // ======================================================== implicit progn of the forms `cur`
BODY:
  if (cur == 0) { v = mkv(K_NIL, 0); goto RET; }
  for (;;) {
    w0 = nword(C, cur);
    a = lo32(w0);
    nxt = hi32(w0);
    ldnode(C, a, at, aw);
    if (nxt == 0) { x = a; t = at; w = aw; d = d + 1; goto EVAL_NODE_LOADED; }   // tail position
    STEP(d + 1);
    if ((at & KIND_MASK) == K_CONS) {
      KPUSH(KF_BODY, nxt, env, vtop, d, 0);
      x = a; t = at; w = aw; d = d + 1;
      goto EVAL_CONS;
    }
    cur = nxt;                                                  // an atom's value is discarded
  }

  // ======================================================== if: cond value v, `cur` = then cell
IF_BRANCH:
  w0 = nword(C, cur);
  if (v.t != K_NIL) { x = lo32(w0); d = d + 1; goto EVAL_NODE; }   // only nil is false (L300-305)
  if (hi32(w0) != 0) { x = car_of(C, hi32(w0)); d = d + 1; goto EVAL_NODE; }
  v = mkv(K_NIL, 0);
  goto RET;

  // ======================================================== return v to the top continuation
RET:
  if (sp == 0) goto done;
  if (VOTE && (__activemask() != R.grp || sp <= R.wait)) {      // diverged, or level with a waiting group
    if (kdirty) *KS(C, sp - 1) = ktop;
    err = E_YIELD;
    goto done;
  }
RET_POP:
  if (NEST && sp == 0) goto done;
  k = ktop;
  --sp;
  if (sp > 0) ktop = *KS(C, sp - 1);                            // consumed at the next return
  kdirty = false;
  kd = kdepth(k.w);
  switch (kkind(k.w)) {
    case KF_ARGS:
      base = k.z; cnt = kcount(k.w);
      hv = *VS(C, base);                                        // needed at APPLY: load early
      if (__builtin_expect(!!(base + 1 + cnt >= vcap), 0)) FAIL(E_OOM);
      *VS(C, base + 1 + cnt) = vpack(v, 0);
      ++cnt;
      cur = k.x; env = k.y; d = kd;
      goto ARGS;
    case KF_IF:
      vtop = k.z; cur = k.x; env = k.y; d = kd;
      goto IF_BRANCH;
    case KF_JOIN: {                                             // argument `cnt + 1` was split off
      base = k.z; cnt = kcount(k.w);
      hv = *VS(C, base);
      if (__builtin_expect(!!(base + 2 + cnt >= vcap), 0)) FAIL(E_OOM);
      *VS(C, base + 1 + cnt) = vpack(v, 0);
      ++cnt;
      cur = k.x; env = k.y; d = kd;
      uint32_t g = hv.z - 1;
      SplitGroup* G = C.A->groups + g;
      uint32_t st = ld_acquire(&G->state);
      if (st == SPLIT_OPEN) {                                   // unclaimed: take the group back
        st = atomicCAS(&G->state, SPLIT_OPEN, SPLIT_TAKEN);
        if (st == SPLIT_OPEN) st = SPLIT_TAKEN;
      }
      if (st == SPLIT_TAKEN) { group_release(*C.A, g); goto ARGS; }   // evaluate the argument here
      SplitTask* T = &G->t[threadIdx.x & 31];
      if (ld_acquire(&T->done) == 0 && !join_wait(*C.A, T, g, form)) goto ARGS;   // gave up: evaluate here
      uint64_t ts = T->rsteps;
      uint32_t te = T->rerr;
      V tv = mkv(T->rt, T->rw);
      group_release(*C.A, g);
      // c.10: the sequential count at the end of this argument is steps + ts; fuel is checked first
      if (te == E_FUEL || steps + ts > fuel) { err = E_FUEL; steps = fuel + 1; goto done; }
      steps += ts;
      if (te) FAIL((uint8_t)te);
      *VS(C, base + 1 + cnt) = vpack(tv, 0);
      ++cnt;
      cur = cdr_of(C, cur);
      goto ARGS;
    }
    case KF_BODY:
      vtop = k.z; cur = k.x; env = k.y; d = kd;
      goto BODY;
    case KF_HEAD:
      cur = k.x; env = k.y; vtop = k.z; d = kd;
      t = 0;                                                    // a computed head: no TAG_VALID
      goto HEAD;
    case KF_LET: goto RET_LET;
    case KF_SETQ: goto RET_SETQ;
    case KF_DEFINE: goto RET_DEFINE;
    case KF_MACRO: goto RET_MACRO;
    case KF_PAR: goto RET_PAR;
    case KF_DATA: goto RET_DATA;
    case KF_QQ: goto RET_QQ;
    default:
      FAIL(E_SYNTAX);
  }

  // ---- cold sections, placed after the hot loop so that its instructions stay contiguous ----
  // ======================================================== returns to the rarer continuations
RET_LET: {

      base = k.z; cnt = kcount(k.w);
      w0 = nword(C, k.x);
      uint32_t sym = (uint32_t)nword(C, car_of(C, lo32(w0)));
      if (__builtin_expect(!!(base + 1 + cnt >= vcap || cnt >= 0x7fffu), 0)) FAIL(E_OOM);
      *VS(C, base + 1 + cnt) = vpack(v, sym);
      ++cnt;
      cur = hi32(w0); env = k.y; d = kd;
      goto LET_LOOP;
}
RET_SETQ: {

      uint8_t e = setq_store(C, k.x, k.y, v);
      if (__builtin_expect(!!(e), 0)) FAIL(e);
      vtop = k.z;
      goto RET;
}
RET_DEFINE: {
      H.gtag[k.x] = (uint8_t)v.t;
      H.gword[k.x] = v.w;
      v = mkv(K_SYM, k.x);
      vtop = k.z;
      goto RET;
}
RET_MACRO: {
      vtop = k.z; env = k.y; d = kd + 1;
      goto EVAL_VALUE;
}
RET_PAR: {
                                              // element i finished
      uint32_t m = kcount(k.w), i = k.x, pb = k.z;
      uint4 st = *VS(C, pb);
      uint32_t spine = st.x, n = st.y;
      uint32_t ca = box_into(H, v, spine + n + i);
      H.tag[spine + i] = K_CONS | TAG_PROPER;
      H.word[spine + i] = pack2(ca, i + 1 < n ? spine + i + 1 : 0);
      if (i + 1 == n) { v = mkv(K_CONS, spine); vtop = pb; goto RET; }
      KPUSH(KF_PAR, i + 1, 0, pb, kd, m);
      goto PAR_NEXT;
}
RET_DATA: {

      base = k.z;
      uint4 st = *VS(C, base);
      uint32_t s = st.x, n = st.y, i = st.z;
      uint32_t ca = box_into(H, v, s + n + i);
      H.tag[s + i] = K_CONS | TAG_PROPER;
      H.word[s + i] = pack2(ca, i + 1 < n ? s + i + 1 : 0);
      cnt = i + 1;
      cur = k.x; env = k.y; d = kd;
      goto DATA_LOOP;
}

  // ======================================================== macro call (c.4 MACRO branch, c.13 #13)
MACRO_CALL: {
    uint64_t mw = nword(C, (uint32_t)v.w);
    uint32_t menv = hi32(mw);
    uint64_t cw = nword(C, lo32(mw));
    uint32_t ps = lo32(cw), body = hi32(cw);
    uint32_t hdr = vtop, n = 0;
    a = cur;
    while (ps != 0 && a != 0) {                                 // bind params to UNevaluated forms
      uint64_t pw = nword(C, ps), aw2 = nword(C, a);
      if (__builtin_expect(!!(hdr + 1 + n >= vcap), 0)) FAIL(E_OOM);
      *VS(C, hdr + 1 + n) = vpack(unbox(C, lo32(aw2)), (uint32_t)nword(C, lo32(pw)));
      ++n;
      ps = hi32(pw);
      a = hi32(aw2);
    }
    if (__builtin_expect(!!(ps != 0 || a != 0), 0)) FAIL(E_ARITY);
    if (__builtin_expect(!!(n >= 0x8000u), 0)) FAIL(E_OOM);
    *VS(C, hdr) = make_uint4(menv, 0, n, K_FRAME);
    KPUSH(KF_MACRO, 0, env, hdr, d, 0);
    env = stack_env(hdr, n);
    if (C.A->mut) MUT_FRAME();
    vtop = hdr + 1 + n;
    cur = body;
    goto BODY;
}

  // ======================================================== data list / (list ...): set up the spine
DATA_START: {
    bool data = v.t != K_BUILTIN;
    uint32_t n = data ? 1 : 0;
    if (NEST) {                                                 // (batches with wide lists run NEST)
      NTRACE_MAX(6);
      const uint4 q0 = cur ? *reinterpret_cast<const uint4*>(H.tag.p + cur) : make_uint4(0, 0, 0, 0);
      if (q0.z & TAG_LEN) {
        n += q0.w;                                              // a reader's wide list: its length, O(1)
      } else {
        uint32_t c = cur;
        for (uint32_t k = 0; k < 16 && c != 0; ++k, ++n) c = cdr_of(C, c); // short lists inline;
        if (c != 0) n += chain_length(C, c);                              // long ones 32 cells per round
      }
      NTRACE_MAX(7);
    } else {
      for (uint32_t c = cur; c != 0; c = cdr_of(C, c)) ++n;
    }
    if (n == 0) { v = mkv(K_NIL, 0); goto RET; }
    uint32_t s;
    if (__builtin_expect(!!(!heap_alloc<!VOTE>(H, 2 * n, &s)), 0)) FAIL(E_OOM);
    if (data) {
      uint32_t ca = box_into(H, v, s + n);
      H.tag[s] = K_CONS | TAG_PROPER;
      H.word[s] = pack2(ca, n > 1 ? s + 1 : 0);
    }
    if (NEST && !APPLY && C.A->nest && n - (data ? 1 : 0) >= WIDE_MIN) {
      // a wide list below the top level (K12 "per warp for wide forms", §8(f)1): suspend; any thread
      // evaluates element i in a heap copy of env (frames are immutable, c.3) into spine cell off + i,
      // then we resume at RET with the spine (steps: the sum over the elements, as in DATA_LOOP)
      uint32_t henv;
      if (__builtin_expect(!!(!promote(C, env, &henv)), 0)) FAIL(E_OOM);
      uint32_t slot = atomicAdd(C.A->nnest, 1u);
      if (slot < C.A->maxnest) {
        NestDesc* D = C.A->ndesc + slot;
        D->form = form;
        D->n = n - (data ? 1 : 0);
        D->m = 0;
        D->spine = s;
        D->ftag = 0;
        D->depth = d;
        D->fword = 0;
        D->steps0 = steps;
        D->top = atomicAdd(H.top, 0ull);
        D->heads[0] = cur;
        D->sp = sp;
        D->vtop = vtop;
        D->kind = NEST_EVAL;
        D->env = henv;
        D->off = data ? 1 : 0;
        D->ncells = n;
        D->total = 0;
        D->bad = 0;
        D->done = 0;
        D->next = 0;
        __threadfence();
        atomicExch(&D->ready, 1u);                              // publish: elements may be claimed
        if (kdirty) *KS(C, sp - 1) = ktop;                      // the resume reloads the top frame
        v = mkv(K_CONS, s);
        aux = slot;
        err = E_SUSPEND;
        goto done;
      }
    }
    if (__builtin_expect(!!(vtop >= vcap), 0)) FAIL(E_OOM);
    base = vtop;
    *VS(C, base) = make_uint4(s, n, 0, 0);                      // {spine, n}
    cnt = data ? 1 : 0;                                         // next element index
    goto DATA_LOOP;
}

  // ======================================================== (||| n f l1 ... lm), c.7
PAR_APPLY: {
    uint32_t n;
    if (fanout && sp == 0 && d == 1 && cnt >= 3 && cnt - 2 <= FANOUT_MAXM) {
      // top-level ||| form: its arguments are evaluated; hand the elements to the fan-out kernel
      // (SURVEY §8(a)6).  Errors decidable now are raised exactly; list lengths are verified by the
      // element kernel (a short or non-contiguous list sends the form to sequential re-evaluation).
      uint8_t e = par_check_light(C, base, cnt, &n);
      if (__builtin_expect(!!(e), 0)) FAIL(e);
      if (n == 0) { v = mkv(K_NIL, 0); vtop = base; goto RET; }
      uint32_t slot = atomicAdd(C.A->npend, 1u);
      if (slot < C.A->maxdesc) {
        uint32_t spine;
        if (__builtin_expect(!!(!heap_alloc<!VOTE>(H, 2 * n, &spine)), 0)) FAIL(E_OOM);
        FanDesc* D = C.A->desc + slot;
        V f = arg(C, base, 1);
        D->form = form;
        D->n = n;
        D->m = cnt - 2;
        D->kind = FAN_PAR;
        D->nelem = n;
        D->spine = spine;
        D->ftag = f.t;
        D->depth = d;
        D->fword = f.w;
        D->steps0 = steps;
        D->top = atomicAdd(H.top, 0ull);
        for (uint32_t j = 0; j < cnt - 2; ++j) D->heads[j] = (uint32_t)arg(C, base, 2 + j).w;
        D->total = 0;
        D->bad = 0;
        D->nonflat = 0;
        err = E_PENDING;
        goto done;
      }
    }
    if (NEST && !APPLY && C.A->nest && cnt >= 3 && cnt - 2 <= FANOUT_MAXM) {
      // nested ||| (§8(f)1): suspend; the elements are applied by any threads, then we resume at RET
      uint8_t e = par_check_light(C, base, cnt, &n);
      if (__builtin_expect(!!(e), 0)) FAIL(e);
      if (n == 0) { v = mkv(K_NIL, 0); vtop = base; goto RET; }
      if (n >= NEST_MIN) {
        uint32_t slot = atomicAdd(C.A->nnest, 1u);
        if (slot < C.A->maxnest) {
          uint32_t spine;
          if (__builtin_expect(!!(!heap_alloc<!VOTE>(H, 2 * n, &spine)), 0)) FAIL(E_OOM);
          NestDesc* D = C.A->ndesc + slot;
          V f = arg(C, base, 1);
          D->form = form;
          D->n = n;
          D->m = cnt - 2;
          D->spine = spine;
          D->ftag = f.t;
          D->depth = d;
          D->fword = f.w;
          D->steps0 = steps;
          D->top = atomicAdd(H.top, 0ull);
          for (uint32_t j = 0; j < cnt - 2; ++j) D->heads[j] = (uint32_t)arg(C, base, 2 + j).w;
          D->sp = sp;
          D->vtop = base;
          D->kind = NEST_APPLY;
          D->total = 0;
          D->bad = 0;
          D->done = 0;
          D->next = 0;
          __threadfence();
          atomicExch(&D->ready, 1u);                            // publish: elements may be claimed
          if (kdirty) *KS(C, sp - 1) = ktop;                    // the resume reloads the top frame
          v = mkv(K_CONS, spine);
          aux = slot;
          err = E_SUSPEND;
          goto done;
        }
      }
    }
    uint8_t e = par_check(C, base, cnt, &n);
    if (__builtin_expect(!!(e), 0)) FAIL(e);
    if (n == 0) { v = mkv(K_NIL, 0); vtop = base; goto RET; }
    uint32_t m = cnt - 2, spine;
    if (__builtin_expect(!!(!heap_alloc<!VOTE>(H, 2 * n, &spine)), 0)) FAIL(E_OOM);
    // state: vs[base] = {spine, n}, vs[base+1] = f, vs[base+2+j] = list cursor j
    V f = arg(C, base, 1);
    for (uint32_t j = 0; j < m; ++j) *VS(C, base + 2 + j) = *VS(C, base + 3 + j);
    *VS(C, base + 1) = vpack(f, 0);
    *VS(C, base) = make_uint4(spine, n, 0, 0);
    KPUSH(KF_PAR, 0, 0, base, d, m);
    goto PAR_NEXT;
}

  // ======================================================== let: binding `cur` next (parallel let)
LET_LOOP:
  while (cur != 0) {
    w0 = nword(C, cur);
    uint64_t bw = nword(C, lo32(w0));
    uint32_t e = car_of(C, hi32(bw));
    ldnode(C, e, at, aw);
    STEP(d + 1);
    V lv;
    if ((at & KIND_MASK) == K_CONS) {
      int leaf;
      TRY_LEAF(leaf, lv);
      if (__builtin_expect(leaf == 2, 0)) goto done;
      if (leaf == 0) {
        vtop = base + 1 + cnt;
        KPUSH(KF_LET, cur, env, base, d, cnt);
        x = e; t = at; w = aw; d = d + 1;
        goto EVAL_CONS;
      }
    } else {
      lv = ATOMVAL(e, at, aw);
    }
    if (__builtin_expect(!!(base + 1 + cnt >= vcap || cnt >= 0x7fffu), 0)) FAIL(E_OOM);
    *VS(C, base + 1 + cnt) = vpack(lv, (uint32_t)nword(C, lo32(bw)));
    ++cnt;
    cur = hi32(w0);
  }
  cur = VS(C, base)->x;                                         // body list stored in the header
  *VS(C, base) = make_uint4(env, 0, cnt, K_FRAME);
  env = stack_env(base, cnt);
  if (C.A->mut) MUT_FRAME();
  vtop = base + 1 + cnt;
  goto BODY;

  // ======================================================== data list / list: element `cnt` next
DATA_LOOP: {
  uint4 st = *VS(C, base);
  uint32_t s = st.x, n = st.y;
  while (cur != 0) {
    w0 = nword(C, cur);
    a = lo32(w0);
    nxt = hi32(w0);
    ldnode(C, a, at, aw);
    STEP(d + 1);
    if ((at & KIND_MASK) == K_CONS) {
      VS(C, base)->z = cnt;
      vtop = base + 1;
      KPUSH(KF_DATA, nxt, env, base, d, 0);
      x = a; t = at; w = aw; d = d + 1;
      goto EVAL_CONS;
    }
    v = ATOMVAL(a, at, aw);
    uint32_t ca = box_into(H, v, s + n + cnt);
    H.tag[s + cnt] = K_CONS | TAG_PROPER;
    H.word[s + cnt] = pack2(ca, cnt + 1 < n ? s + cnt + 1 : 0);
    ++cnt;
    cur = nxt;
  }
  vtop = base;
  v = mkv(K_CONS, s);
  goto RET;
}

  // ======================================================== quasiquote template walk (R8)
  // QQ_NODE: template node x at level qlev; its value returns to the top continuation.  A template list is
  // rebuilt on the V-stack (header at base: element count when a KF_QQ frame is pushed; elements above)
  // and then copied into a fresh contiguous spine.  d stays the quasiquote form's depth; unquoted
  // expressions are evaluated at d + 1.  The walk itself takes no steps.
QQ_SPECIAL:                                                     // (quasiquote t); unquote forms: SYNTAX
  if (v.w != SP_QUASIQUOTE) FAIL(E_SYNTAX);                     // only meaningful inside a template
  x = car_of(C, cur);
  qlev = 1;
  // fallthrough
QQ_NODE: {
    uint32_t tt;
    uint64_t tw;
    ldnode(C, x, tt, tw);
    if ((tt & KIND_MASK) != K_CONS) { v = unbox_loaded(x, tt, tw); goto RET; }
    if (__builtin_expect(!!(!(tt & TAG_PROPER)), 0)) FAIL(E_SYNTAX);
    uint32_t op = qq_op(C, tw), arg = 0;
    if (op == SP_UNQUOTE && qlev == 1) {
      if (!qq_arg(C, tw, &arg)) FAIL(E_SYNTAX);
      x = arg; d = d + 1;
      goto EVAL_NODE;                                           // (tail: the value returns to our caller)
    }
    if (op == SP_UNQUOTE_SPLICING && qlev == 1) FAIL(E_SYNTAX);   // not in an element position
    hop = qlev;                                                 // level of the elements after the head
    if (op != 0xffu) {
      if (!qq_arg(C, tw, &arg)) FAIL(E_SYNTAX);
      hop = op == SP_QUASIQUOTE ? qlev + 1 : qlev - 1;
    }
    if (__builtin_expect(!!(vtop >= vcap), 0)) FAIL(E_OOM);
    base = vtop;
    vtop = base + 1;
    cur = x;
    goto QQ_LIST;
}
QQ_LIST:                                                        // element `cur` next, at level qlev
  while (cur != 0) {
    w0 = nword(C, cur);
    a = lo32(w0);
    nxt = hi32(w0);
    ldnode(C, a, at, aw);
    if ((at & KIND_MASK) != K_CONS) {                           // an atom: itself
      if (__builtin_expect(!!(vtop >= vcap), 0)) FAIL(E_OOM);
      *VS(C, vtop) = vpack(unbox_loaded(a, at, aw), 0);
      ++vtop;
      cur = nxt;
      qlev = hop;
      continue;
    }
    VS(C, base)->x = vtop - base - 1;                           // elements so far
    if (qlev == 1 && qq_op(C, aw) == SP_UNQUOTE_SPLICING) {     // evaluate, then splice
      uint32_t arg;
      if (!(at & TAG_PROPER) || !qq_arg(C, aw, &arg)) FAIL(E_SYNTAX);
      KPUSH(KF_QQ, nxt, env, base, d, hop | 0x100u);
      x = arg; d = d + 1;
      goto EVAL_NODE;
    }
    KPUSH(KF_QQ, nxt, env, base, d, hop);                       // a sub-template
    x = a;
    goto QQ_NODE;
  }
  {
    uint32_t n = vtop - base - 1, s;
    if (n == 0) {
      v = mkv(K_NIL, 0);
    } else {
      if (__builtin_expect(!!(!heap_alloc<!VOTE>(H, 2 * n, &s)), 0)) FAIL(E_OOM);
      for (uint32_t i = 0; i < n; ++i) {
        uint32_t ca = box_into(H, vunpack(*VS(C, base + 1 + i)), s + n + i);
        H.tag[s + i] = K_CONS | TAG_PROPER;
        H.word[s + i] = pack2(ca, i + 1 < n ? s + i + 1 : 0);
      }
      v = mkv(K_CONS, s);
    }
    vtop = base;
    goto RET;
  }
RET_QQ: {                                                       // an element's value (or a list to splice)
    base = k.z;
    cur = k.x; env = k.y; d = kd;
    hop = kcount(k.w) & 0xffu;
    qlev = hop;
    vtop = base + 1 + VS(C, base)->x;
    if (kcount(k.w) & 0x100u) {
      if (__builtin_expect(!!(!proper_value(C, v)), 0)) FAIL(E_TYPE);
      for (uint32_t c = v.t == K_NIL ? 0 : (uint32_t)v.w; c != 0; c = cdr_of(C, c)) {
        if (__builtin_expect(!!(vtop >= vcap), 0)) FAIL(E_OOM);
        *VS(C, vtop) = vpack(unbox(C, car_of(C, c)), 0);
        ++vtop;
      }
    } else {
      if (__builtin_expect(!!(vtop >= vcap), 0)) FAIL(E_OOM);
      *VS(C, vtop) = vpack(v, 0);
      ++vtop;
    }
    goto QQ_LIST;
}

  // ======================================================== ||| : start element i (frame in ktop)
PAR_NEXT: {
  uint32_t m = kcount(ktop.w), pb = ktop.z;
  V f = vunpack(*VS(C, pb + 1));
  base = pb + 2 + m;
  if (__builtin_expect(!!(base + 1 + m >= vcap), 0)) FAIL(E_OOM);
  hv = vpack(f, 0);
  *VS(C, base) = hv;
  for (uint32_t j = 0; j < m; ++j) {
    uint4* cj = VS(C, pb + 2 + j);
    uint64_t wj = nword(C, cj->x);
    *VS(C, base + 1 + j) = vpack(unbox(C, lo32(wj)), 0);
    cj->x = hi32(wj);
  }
  cnt = m;
  vtop = base + 1 + m;
  d = kdepth(ktop.w);
  goto APPLY;
}


done:
  if (SPLIT && err != 0 && err != E_PENDING && err != E_SUSPEND && sp > 0) abandon_joins(C, sp, ktop);
#undef FAIL
#undef STEP
#undef KPUSH
#undef ATOMVAL
  FormOut o;
  o.t = v.t;
  o.w = v.w;
  o.steps = steps;
  o.err = err;
  o.aux = aux;
  if (VOTE && err == E_YIELD) {
    o.aux = sp;
    o.vtop = vtop;
    o.kk = kkind(ktop.w);
  }
  return o;
}

}  // namespace culi
