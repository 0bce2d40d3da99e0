// culi_kernels.cu — sm_100a kernels of libculi.so: image relocation, batch eval (one thread per form,
// warps take consecutive forms of the binned order), define (sequential), result export.
// The eval/apply machine itself is culi_machine.cuh.
#include <cuda_runtime.h>
#include <stdint.h>

#include "culi_machine.cuh"

namespace culi {

// Relocate an uploaded image into the heap: image-local indices -> heap indices, and
// interleave the image's tag[] / word[] arrays (staged in HBM) into 16-byte nodes (one store per node).
__global__ void culi_relocate_kernel(const uint8_t* __restrict__ stag, const uint64_t* __restrict__ sword,
                                     Node* nodes, uint64_t base, uint64_t n,
                                     uint32_t str_base, uint32_t* roots, uint32_t nroots) {
  uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
    uint64_t g = base + i;
    uint32_t tg = stag[i], t = tg & KIND_MASK;
    uint64_t w = sword[i];
    if (t == K_CONS) {
      uint32_t a = lo32(w), b = hi32(w);
      a = a < IMG_FIRST ? a : (uint32_t)(base + a - IMG_FIRST);
      b = b < IMG_FIRST ? b : (uint32_t)(base + b - IMG_FIRST);
      w = pack2(a, b);
    } else if (t == K_STR) {
      w = pack2(lo32(w) + str_base, hi32(w));
    }
    *reinterpret_cast<uint4*>(nodes + g) = make_uint4(lo32(w), hi32(w), tg, 0);
  }
  for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < nroots; i += stride) {
    uint32_t r = roots[i];
    roots[i] = r < IMG_FIRST ? r : (uint32_t)(base + r - IMG_FIRST);
  }
}

// Mark the second cell of every wide list of an uploaded image with its remaining length (TAG_LEN): pairs of
// (image-local cell, cells from it to the end), relocated to base.  One writer per cell.
__global__ void culi_lenmark_kernel(Node* nodes, uint64_t base, const uint32_t* pairs, uint32_t npairs) {
  for (uint32_t k = blockIdx.x * blockDim.x + threadIdx.x; k < npairs; k += gridDim.x * blockDim.x) {
    Node* x = nodes + base + (pairs[2 * k] - IMG_FIRST);
    x->len = pairs[2 * k + 1];
    x->tag = (uint8_t)(x->tag | TAG_LEN);
  }
}
cudaError_t launch_lenmark(cudaStream_t s, Node* nodes, uint64_t base, const uint32_t* pairs, uint32_t npairs) {
  culi_lenmark_kernel<<<(npairs + 255) / 256, 256, 0, s>>>(nodes, base, pairs, npairs);
  return cudaGetLastError();
}

__device__ __forceinline__ void write_result(const EvalArgs& A, uint32_t f, const FormOut& o) {
  A.rtag[f] = o.err ? (uint8_t)K_ERROR : (uint8_t)o.t;
  A.rerr[f] = o.err;
  A.rsteps[f] = o.steps;
  A.rword[f] = o.w;
  if (o.err == E_OOM) atomicExch(&A.flags[0], 1);   // (E_PENDING: filled in by the fan-out finalizer)
}

__device__ __forceinline__ Ctx make_ctx(const EvalArgs& A, uint32_t slot) {
  Ctx C;
  C.A = &A;
  C.kb = A.kst + slot;
  C.vb = A.vst + slot;
  return C;
}

// ---- nested |||: claim and apply one element of descriptor D ---------------------------
// Runs on the thread's secondary stacks (C2).  Element i: f applied to (l1[i] .. lm[i]) at the depth of the
// ||| call, with the fuel left when the owner suspended.  A failed contiguity check or an element error
// marks the descriptor bad (the owner's form is then re-evaluated sequentially, exactly).

#if CULI_NEST_TRACE
extern "C" int culi_debug_nest_trace(unsigned long long* out) { return culi_nest_trace_read(out); }
extern "C" int culi_debug_nest_trace_reset() { return culi_nest_trace_reset(); }
#endif
__device__ __forceinline__ bool nest_run_one(const EvalArgs& A, const Ctx& C2, NestDesc* D) {
  if (*(volatile uint32_t*)&D->ready == 0) return false;
  uint32_t n = D->n;
  if (*(volatile uint32_t*)&D->next >= n) return false;
  uint32_t i = fetch_add_grouped(&D->next);           // (one atomic per warp and descriptor)
  if (i >= n) return false;
  NTRACE_MIN(0);
  if (CULI_NEST_TRACE == 1) NTRACE_ADD(4, 1);
  const DevHeap& H = A.H;
  uint32_t m = D->m, spine = D->spine;
  bool ok = true;
  if (D->kind == NEST_EVAL) {                           // wide list: evaluate element expression i
    uint32_t c = D->heads[0] + i, nc = D->ncells, cell = D->off + i;
    uint32_t tc = H.tag[c];
    uint64_t wc = H.word[c];
    if ((uint64_t)c >= D->top || (tc & KIND_MASK) != K_CONS || (i + 1 < n && hi32(wc) != c + 1)) {
      atomicOr(&D->bad, 1u);
    } else {
      FormOut o = eval_form<false, false>(C2, lo32(wc), D->form, 0, 0, A.fuel - D->steps0, D->depth + 1,
                                          false, Resume{}, D->env);
      if (o.err) {
        atomicOr(&D->bad, 2u);
      } else {
        uint32_t ca = box_into(H, mkv(o.t, o.w), spine + nc + cell);
        H.tag[spine + cell] = K_CONS | TAG_PROPER;
        H.word[spine + cell] = pack2(ca, cell + 1 < nc ? spine + cell + 1 : 0);
        atomicAdd(&D->total, (unsigned long long)o.steps);
      }
    }
    __threadfence();
    atomicAdd(&D->done, 1u);
    NTRACE_MAX(1);
    return true;
  }
  *VS(C2, 0) = vpack(mkv(D->ftag, D->fword), 0);
  for (uint32_t j = 0; j < m; ++j) {
    uint32_t c = D->heads[j] + i;
    if ((uint64_t)c >= D->top) { ok = false; break; }
    uint32_t tc = H.tag[c];
    uint64_t wc = H.word[c];
    if ((tc & KIND_MASK) != K_CONS || (i + 1 < n && hi32(wc) != c + 1)) { ok = false; break; }
    *VS(C2, 1 + j) = vpack(unbox(C2, lo32(wc)), 0);
  }
  if (!ok) {
    atomicOr(&D->bad, 1u);
  } else {
    FormOut o = eval_form<false, true>(C2, 0, D->form, 1, m, A.fuel - D->steps0, D->depth);
    if (o.err) {
      atomicOr(&D->bad, 2u);
    } else {
      uint32_t ca = box_into(H, mkv(o.t, o.w), spine + n + i);
      H.tag[spine + i] = K_CONS | TAG_PROPER;
      H.word[spine + i] = pack2(ca, i + 1 < n ? spine + i + 1 : 0);
      atomicAdd(&D->total, (unsigned long long)o.steps);
    }
  }
  __threadfence();
  atomicAdd(&D->done, 1u);
  return true;
}

// Help any published descriptor with unclaimed elements; returns whether an element was applied.
__device__ __forceinline__ bool nest_help_any(const EvalArgs& A, const Ctx& C2, NestDesc* prefer) {
  if (prefer && nest_run_one(A, C2, prefer)) return true;
  uint32_t nn = *(volatile uint32_t*)A.nnest;
  if (nn > A.maxnest) nn = A.maxnest;
  for (uint32_t k = 0; k < nn; ++k)
    if (nest_run_one(A, C2, A.ndesc + k)) return true;
  return false;
}

// ---- argument splitting: a warp with no form left steals ----------------------------
// Its lanes, once every lane of the warp is idle, work in rounds, coordinated through shared memory only
// (no warp intrinsic: lanes of a warp in different spin loops must never meet in a collective): each lane
// arrives at the warp's round counter; the last to arrive is the round's leader, takes ticket h = head++,
// waits for the entry stamped h and claims its group (OPEN -> CLAIMED) unless the owners took it back
// first, then publishes the result in the warp's mailbox and bumps the round generation; the others wait
// for the generation.  All 32 lanes are in every round, so lane i runs task i of the group (owner lane i's
// argument: converged, like the owners).  Returns the group, 0xfffffffe for no group this round, or
// 0xffffffff once every form of the batch is finished.  Waits back off exponentially (A.split_sleep ns).
__shared__ uint32_t culi_warp_idle[4];       // lanes of each warp with no form left (kernel prologue: 0)
__shared__ uint32_t culi_warp_round[4];      // arrivals at the idle warps' round barrier
__shared__ uint32_t culi_warp_gen[4];        // rounds whose group is in the mailbox
__shared__ uint32_t culi_warp_mail[4];       // the round's group (or 0xfffffffe / 0xffffffff)

__device__ __noinline__ uint32_t claim_group(const EvalArgs& A) {
  SplitCtl* Q = A.sctl;
  unsigned long long h = atomicAdd(&Q->head, 1ull);
  const unsigned long long* qe = &A.gqueue[h & (A.gqcap - 1)];
  uint32_t ns = 64;
  for (uint32_t spin = 0;; ++spin) {
    unsigned long long e = ld_relaxed64(qe);             // (relaxed: an acquire poll invalidates L1)
    if ((uint32_t)(e >> 32) == (uint32_t)h && (uint32_t)e != 0) {   // (0: never written)
      uint32_t g = (uint32_t)e - 1;
      if (atomicCAS(&A.groups[g].state, SPLIT_OPEN, SPLIT_CLAIMED) != SPLIT_OPEN) return 0xfffffffeu;
      A.groups[g].claimer = my_slot() >> 5;
      atomicAdd(&Q->claimed, 1u);
      return g;
    }
    if ((spin & 7) == 0 && *(volatile uint32_t*)A.finished >= A.nforms) return 0xffffffffu;
#if CULI_WATCHDOG
    if (gtime() - *(volatile unsigned long long*)&Q->t0 > (unsigned long long)CULI_WATCHDOG * 1000000ull + 2000000000ull) {
      if (atomicAdd(&Q->wd[0], 1u) == 0) { Q->wd[6] = 1; Q->wd[7] = *(volatile uint32_t*)A.finished; }
      return 0xffffffffu;
    }
#endif
    __nanosleep(ns);
    ns = ns * 2 > A.split_sleep ? A.split_sleep : ns * 2;
  }
}

__device__ __noinline__ uint32_t split_claim(const EvalArgs& A, uint32_t& round) {
  uint32_t w = threadIdx.x >> 5;
  uint32_t r = ++round;
  // wait until the whole warp is idle (the first round only has to)
  for (uint32_t ns = 64; A.steal_gate && *(volatile uint32_t*)&culi_warp_idle[w] < 32;) {
    if (*(volatile uint32_t*)A.finished >= A.nforms) return 0xffffffffu;
    __nanosleep(ns);
    ns = ns * 2 > A.split_sleep ? A.split_sleep : ns * 2;
  }
  if (atomicAdd(&culi_warp_round[w], 1u) == 32u * r - 1u) {   // last to arrive: this round's leader
    uint32_t g = claim_group(A);
    *(volatile uint32_t*)&culi_warp_mail[w] = g;
    __threadfence_block();
    *(volatile uint32_t*)&culi_warp_gen[w] = r;
    return g;
  }
  for (uint32_t ns = 64; *(volatile uint32_t*)&culi_warp_gen[w] < r;) {
    // (a lane that found every form finished leaves without arriving: so does everyone after it)
    if (*(volatile uint32_t*)A.finished >= A.nforms) return 0xffffffffu;
    __nanosleep(ns);
    ns = ns * 2 > A.split_sleep ? A.split_sleep : ns * 2;
  }
  __threadfence_block();
  return *(volatile uint32_t*)&culi_warp_mail[w];
}

// Batch mode.  Shared memory per block: the persistent code segment [code_lo, code_lo + code_n) as
// {w.lo, w.hi, tag, 0} and the global frame [0, gst) ("stage").  Every lane takes its next
// form with a warp-aggregated counter (converged lanes of the binned order get consecutive forms) and runs
// it to completion; no warp-wide barrier anywhere, so diverged lanes never wait on each other.  With SPLIT,
// a lane that finds no form left is a thief: it evaluates split-off arguments of busy lanes on its own
// stacks (one eval_form call site serves forms and tasks).
template <bool FANOUT, bool NEST, bool SPLIT>
__global__ void __launch_bounds__(128, (NEST || SPLIT) ? CULI_SPLIT_BLOCKS_PER_SM : CULI_BLOCKS_PER_SM)
culi_eval_kernel(const __grid_constant__ EvalArgs A) {
  uint4* scode = culi_smem;
  uint64_t* sgword = reinterpret_cast<uint64_t*>(culi_smem + A.code_n);
  uint8_t* sgtag = reinterpret_cast<uint8_t*>(sgword + A.gst);
  for (uint32_t i = threadIdx.x; i < A.code_n; i += blockDim.x) {
    uint64_t w = A.H.word[A.code_lo + i];
    scode[i] = make_uint4(lo32(w), hi32(w), A.H.tag[A.code_lo + i], 0);
  }
  for (uint32_t i = threadIdx.x; i < A.gst; i += blockDim.x) {
    sgword[i] = A.H.gword[i];
    sgtag[i] = A.H.gtag[i];
  }
  alloc_init();
  if (SPLIT && threadIdx.x < 4) {
    culi_split_busy[threadIdx.x] = 0;
    culi_warp_idle[threadIdx.x] = 0;
    culi_warp_round[threadIdx.x] = 0;
    culi_warp_gen[threadIdx.x] = 0;
  }
  __syncthreads();
  uint32_t slot = my_slot();
  Ctx C = make_ctx(A, slot);
  Ctx C2;
  if (NEST) {
    C2.A = &A;
    C2.kb = A.kst2 + slot;
    C2.vb = A.vst2 + slot;
  }
  bool forms_left = true;
  if (!SPLIT && !NEST && (threadIdx.x & 31) >= A.lanes) return;   // thin warps for small batches
  if (NEST && threadIdx.x == 0) NTRACE_MIN(5);
  uint32_t round = 0;                                   // idle rounds taken (split_claim)
  SplitGroup* G = nullptr;                              // the claimed group whose tasks this lane runs
  uint32_t todo = 0;                                    // its task positions left for this lane
  for (;;) {
    uint32_t f = 0, root = 0, env = 0, d = 1;
    uint64_t fuel = A.fuel;
    SplitTask* T = nullptr;
    if (!SPLIT || forms_left) {
      uint32_t i = fetch_add_lanes32(A.next);
      if (i >= A.nforms) {
        if (!SPLIT) break;
        forms_left = false;
        atomicAdd(&culi_warp_idle[threadIdx.x >> 5], 1u);
        continue;
      }
      f = A.perm ? A.perm[i] : i;
      root = A.roots[f];
    } else {
      if (!todo) {
        uint32_t g = split_claim(A, round);
        if (g == 0xffffffffu) break;
        if (g == 0xfffffffeu) continue;
        G = A.groups + g;
        ld_acquire(&G->state);                          // acquire the owners' task and env writes
        todo = G->mask & (1u << (threadIdx.x & 31));   // lane i runs owner lane i's task
        if (!todo) continue;
      }
      uint32_t p = __ffs(todo) - 1;
      todo &= todo - 1;
      T = &G->t[p];
      f = G->form;
      root = T->expr;
      env = T->env;
      d = T->depth;
      fuel = T->budget;
    }
    FormOut o;
    bool resume = false;
    Resume R{};
    for (;;) {
      o = eval_form<FANOUT, false, NEST, SPLIT>(C, root, f, 0, 0, fuel, d, resume, R, env);
      if (!NEST || o.err != E_SUSPEND) break;
      NestDesc* D = A.ndesc + o.aux;                    // suspended on a nested |||: help until done
      NTRACE_MIN(3);
      unsigned long long t0 = 0;
      while (*(volatile uint32_t*)&D->done < D->n) {
        if (nest_help_any(A, C2, D)) { t0 = 0; continue; }
        __nanosleep(128);
        unsigned long long now = gtime();                     // bounded: an element that never finishes
        if (!t0) t0 = now;                                    // sends the form to the sequential fallback
        else if (now - t0 > A.wait_ns) { wait_gave_up(A, WAIT_NEST, o.aux, f); atomicOr(&D->bad, 4u); break; }
      }
      __threadfence();
      uint64_t s = D->steps0 + *(volatile unsigned long long*)&D->total;
      if (*(volatile uint32_t*)&D->bad || s > A.fuel) {   // decide exactly: sequential re-evaluation
        A.fallback[atomicAdd(A.nfallback, 1u)] = f;
        o.err = E_PENDING;
        break;
      }
      NTRACE_MAX(2);
      R.sp = D->sp;
      R.vtop = D->vtop;
      R.steps = s;
      R.v = mkv(K_CONS, D->spine);
      resume = true;
    }
    if (SPLIT && T) {                                   // a split-off argument: hand it to its owner
      T->rt = o.t;
      T->rw = o.w;
      T->rsteps = o.steps;
      T->rerr = o.err;
      st_release(&T->done, 1u);                         // (the release orders the result writes)
    } else {
      write_result(A, f, o);
      if (NEST || SPLIT) atomicAdd(A.finished, 1u);
    }
  }
  if (NEST) {                                           // no forms left: help until every form is done
    uint32_t ns = 128;                                  // (back off while there is nothing to claim: the
    while (*(volatile uint32_t*)A.finished < A.nforms) {  //  whole grid polls the same descriptors; longer
      if (nest_help_any(A, C2, nullptr)) { ns = 128; continue; }   // before the first one is published)
      __nanosleep(ns);
      uint32_t cap = *(volatile uint32_t*)A.nnest ? 2048u : 8192u;
      ns = ns * 2 > cap ? cap : ns * 2;
    }
  }
}

// Batch mode with warp voting (north_star: "ballot for branch voting").  Divergence is the
// cost the paper names for SIMT evaluation of different forms (§III-D.d).  A warp takes 32
// forms; the lanes start together; a lane group that diverges yields at its next return (E_YIELD, its
// state saved); the warp then votes: every waiting lane offers key = stack height << 4 | kind of the
// continuation it is about to pop, __reduce_max_sync picks the deepest, and the lanes with that key are
// resumed together (same height and same continuation: the same place of the same-shaped form).  The
// group runs until it diverges again or returns down to the height of the deepest other waiting lane,
// where the groups merge.  Used for batches that neither split arguments nor nest |||.
template <bool FANOUT>
__global__ void __launch_bounds__(128, CULI_BLOCKS_PER_SM) culi_eval_vote_kernel(const __grid_constant__ EvalArgs A) {
  uint64_t* sgword = reinterpret_cast<uint64_t*>(culi_smem);
  uint8_t* sgtag = reinterpret_cast<uint8_t*>(sgword + A.gst);
  for (uint32_t i = threadIdx.x; i < A.gst; i += blockDim.x) {
    sgword[i] = A.H.gword[i];
    sgtag[i] = A.H.gtag[i];
  }
  alloc_init();
  __syncthreads();
  uint32_t slot = blockIdx.x * blockDim.x + threadIdx.x;
  Ctx C = make_ctx(A, slot);
  int lane = threadIdx.x & 31;
  for (;;) {
    uint32_t b = 0;
    if (lane == 0) b = atomicAdd(A.next, 32u);
    b = __shfl_sync(0xffffffffu, b, 0);
    if (b >= A.nforms) break;
    uint32_t i = b + lane, f = 0, root = 0, key = 0;
    bool live = i < A.nforms, fresh = true;
    if (live) {
      f = A.perm ? A.perm[i] : i;
      root = A.roots[f];
    }
    Resume R{};
    R.grp = __ballot_sync(0xffffffffu, live);                  // first: every lane from its root
    R.wait = 0;
    for (;;) {
      if ((R.grp >> lane) & 1u) {
        FormOut o = eval_form<FANOUT, false, false, false, true>(C, root, f, 0, 0, A.fuel, 1, !fresh, R);
        fresh = false;
        if (o.err == E_YIELD) {
          R.sp = o.aux;
          R.vtop = o.vtop;
          R.steps = o.steps;
          R.v = mkv(o.t, o.w);
          key = (o.aux << 4) | o.kk;
        } else {
          write_result(A, f, o);
          live = false;
        }
      }
      __syncwarp();
      uint32_t mykey = live ? key : 0u;
      uint32_t best = __reduce_max_sync(0xffffffffu, mykey);
      if (best == 0) break;                                     // every lane's form is finished
      unsigned grp = __ballot_sync(0xffffffffu, live && mykey == best);
      uint32_t wait = __reduce_max_sync(0xffffffffu, (live && mykey != best) ? (key >> 4) : 0u);
      if ((grp >> lane) & 1u) { R.grp = grp; R.wait = wait; }
      else R.grp = grp;                                         // (not resumed: only the membership test)
    }
  }
}

// Define mode (culi_define): forms evaluated in order by one thread; define/defun/defmacro write the
// global frame; stops at the first error.  No staging: this kernel writes globals.
__global__ void culi_define_kernel(const __grid_constant__ EvalArgs A) {
  if (blockIdx.x != 0 || threadIdx.x != 0) return;
  alloc_init();
  Ctx C = make_ctx(A, 0);
  for (uint32_t f = 0; f < A.nforms; ++f) {
    FormOut o = eval_form<false, false>(C, A.roots[f], f, 0, 0, A.fuel);
    write_result(A, f, o);
    if (o.err) {
      A.flags[1] = (int)f + 1;
      A.flags[2] = o.err;
      return;
    }
  }
}

// Export: serialize every CONS/STR result into pre-order tokens {word, tag}; the
// record's word becomes offset | count << 32.  The thread's V-stack is the DFS stack.
__global__ void __launch_bounds__(128) culi_export_kernel(ExportArgs X) {
  uint32_t slot = blockIdx.x * blockDim.x + threadIdx.x;
  uint32_t nthreads = gridDim.x * blockDim.x;
  uint32_t total = X.list ? X.nlist : X.nforms;
  for (uint32_t q = slot; q < total; q += nthreads) {
    uint32_t f = X.list ? X.list[q] : q;
    uint32_t t = X.rtag[f];
    if (t != K_CONS && t != K_STR) continue;
    uint32_t root = (uint32_t)X.rword[f];
    unsigned long long ntok = 0;
    uint32_t sp = 0, n = root;
    bool ovf = false;
    for (;;) {                                     // pass 1: count tokens
      ++ntok;
      if ((X.tag[n] & KIND_MASK) == K_CONS) {
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
    n = root;
    sp = 0;
    unsigned long long k = off;
    for (;;) {                                     // pass 2: write tokens
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

__global__ void culi_reset_kernel(unsigned long long* top, unsigned long long top_value, uint32_t* next,
                                  unsigned long long* pcount, int* flags, uint32_t* npend,
                                  uint32_t* nfallback, uint32_t* nnest, SplitCtl* sctl) {
  *top = top_value;
  if (sctl) {                                         // tickets continue; unclaimed entries are dropped
    unsigned long long t = sctl->tail > sctl->head ? sctl->tail : sctl->head;
    sctl->head = t;
    sctl->tail = t;
    sctl->published = 0;
    sctl->claimed = 0;
    for (int k = 0; k < 4; ++k) sctl->stat[k] = 0;
    sctl->timeouts = 0;
    for (int k = 0; k < 9; ++k) sctl->diag[k] = 0;
    for (int k = 0; k < 8; ++k) sctl->wd[k] = 0;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(sctl->t0));
  }
  *next = 0;
  *pcount = 0;
  *npend = 0;
  *nfallback = 0;
  *nnest = 0;                                         // nnest[1] counts finished forms
  nnest[1] = 0;
  for (int k = 0; k < 8; ++k) flags[k] = 0;
}

__global__ void culi_nest_clear_kernel(NestDesc* d, uint32_t n) {
  for (uint32_t k = blockIdx.x * blockDim.x + threadIdx.x; k < n; k += gridDim.x * blockDim.x) d[k].ready = 0;
}

cudaError_t launch_nest_clear(cudaStream_t s, NestDesc* d, uint32_t n) {
  culi_nest_clear_kernel<<<(n + 255) / 256, 256, 0, s>>>(d, n);
  return cudaGetLastError();
}

// ---- ||| fan-out ------------------------------------------------
// Element i of every pending descriptor is applied by one thread: f applied to (l1[i] .. lm[i]) at the
// depth of the ||| form + 1, with the fuel left after the ||| arguments.  Lists are indexed in O(1)
// through their contiguous spines (SURVEY c.14): cell i of list j is heads[j] + i, which the thread
// verifies (cons, inside the heap as it was when the descriptor was written, linked to cell i+1); a
// failed check or an element error marks the form for exact sequential re-evaluation.  Results go to
// the preallocated spine (cells [spine, spine+n), boxes [spine+n, spine+2n)): coalesced stores.
__global__ void __launch_bounds__(128, CULI_BLOCKS_PER_SM) culi_fanout_kernel(const __grid_constant__ EvalArgs A) {
  uint4* scode = culi_smem;
  uint64_t* sgword = reinterpret_cast<uint64_t*>(culi_smem + A.code_n);
  uint8_t* sgtag = reinterpret_cast<uint8_t*>(sgword + A.gst);
  for (uint32_t i = threadIdx.x; i < A.code_n; i += blockDim.x) {
    uint64_t w = A.H.word[A.code_lo + i];
    scode[i] = make_uint4(lo32(w), hi32(w), A.H.tag[A.code_lo + i], 0);
  }
  for (uint32_t i = threadIdx.x; i < A.gst; i += blockDim.x) {
    sgword[i] = A.H.gword[i];
    sgtag[i] = A.H.gtag[i];
  }
  alloc_init();
  __syncthreads();
  uint32_t slot = blockIdx.x * blockDim.x + threadIdx.x;
  uint32_t nthreads = gridDim.x * blockDim.x;
  Ctx C = make_ctx(A, slot);
  uint32_t npend = *A.npend;
  if (npend > A.maxdesc) npend = A.maxdesc;
  const DevHeap& H = A.H;
  for (uint32_t k = 0; k < npend; ++k) {
    FanDesc* D = A.desc + k;
    uint32_t n = D->n, m = D->m, spine = D->spine;
    uint64_t top = D->top;
    V f = mkv(D->ftag, D->fword);
    uint64_t budget = A.fuel - D->steps0;
    unsigned long long my_steps = 0;
    uint32_t bad = 0, nonflat = 0;
    if (D->kind != FAN_PAR) {                         // wide form: element i = argument i (depth 2)
      uint32_t ne = D->nelem, first = D->kind == FAN_DATA ? 1u : 0u, c1 = D->heads[0];
      for (uint32_t i = slot; i < ne; i += nthreads) {
        uint32_t c = c1 + i;
        if ((uint64_t)c >= top) { bad |= 1; continue; }
        uint32_t tc = H.tag[c];
        uint64_t wc = H.word[c];
        if ((tc & KIND_MASK) != K_CONS || hi32(wc) != (i + 1 < ne ? c + 1 : 0u)) { bad |= 1; continue; }
        FormOut o = eval_form<false, false>(C, lo32(wc), D->form, 0, 0, budget, D->depth + 1);
        if (o.err) { bad |= 2; continue; }
        my_steps += o.steps;
        if (D->kind == FAN_FOLD) {                   // raw value record for the finalizer's fold
          H.tag[spine + i] = (uint8_t)o.t;
          H.word[spine + i] = o.w;
          continue;
        }
        nonflat |= (o.t == K_CONS);
        uint32_t j = first + i;
        uint32_t ca = box_into(H, mkv(o.t, o.w), spine + n + j);
        H.tag[spine + j] = K_CONS | TAG_PROPER;
        H.word[spine + j] = pack2(ca, j + 1 < n ? spine + j + 1 : 0);
      }
    } else
    for (uint32_t i = slot; i < n; i += nthreads) {
      bool ok = true;
      *VS(C, 0) = vpack(f, 0);
      for (uint32_t j = 0; j < m; ++j) {
        uint32_t c = D->heads[j] + i;
        if ((uint64_t)c >= top) { ok = false; break; }
        uint32_t tc = H.tag[c];
        uint64_t wc = H.word[c];
        if ((tc & KIND_MASK) != K_CONS || (i + 1 < n && hi32(wc) != c + 1)) { ok = false; break; }
        *VS(C, 1 + j) = vpack(unbox(C, lo32(wc)), 0);
      }
      if (!ok) { bad |= 1; continue; }
      FormOut o = eval_form<false, true>(C, 0, D->form, 1, m, budget);
      if (o.err) { bad |= 2; continue; }
      my_steps += o.steps;
      nonflat |= (o.t == K_CONS);
      uint32_t ca = box_into(H, mkv(o.t, o.w), spine + n + i);
      H.tag[spine + i] = K_CONS | TAG_PROPER;
      H.word[spine + i] = pack2(ca, i + 1 < n ? spine + i + 1 : 0);
    }
    // warp-reduce, one atomic per warp
    for (int o = 16; o > 0; o >>= 1) {
      my_steps += __shfl_down_sync(0xffffffffu, my_steps, o);
      bad |= __shfl_down_sync(0xffffffffu, bad, o);
      nonflat |= __shfl_down_sync(0xffffffffu, nonflat, o);
    }
    if ((threadIdx.x & 31) == 0) {
      if (my_steps) atomicAdd(&D->total, my_steps);
      if (bad) atomicOr(&D->bad, bad);
      if (nonflat) atomicOr(&D->nonflat, 1u);
    }
  }
}

// One thread per descriptor: write the ||| form's record, or queue it for sequential re-evaluation.
__global__ void culi_fanout_finalize_kernel(const __grid_constant__ EvalArgs A) {
  uint32_t npend = *A.npend;
  if (npend > A.maxdesc) npend = A.maxdesc;
  for (uint32_t k = blockIdx.x * blockDim.x + threadIdx.x; k < npend; k += gridDim.x * blockDim.x) {
    const FanDesc* D = A.desc + k;
    uint64_t steps = D->steps0 + D->total;
    if (D->bad || steps > A.fuel) {
      A.fallback[atomicAdd(A.nfallback, 1u)] = D->form;
      continue;
    }
    A.rerr[D->form] = 0;
    A.rsteps[D->form] = steps;
    if (D->kind == FAN_FOLD) {                        // (+ / * a1 .. an): types, then left fold (c.6)
      bool type_err = false;
      for (uint32_t i = 0; i < D->nelem; ++i) type_err |= !is_num(A.H.tag[D->spine + i]);
      if (type_err) {
        A.rtag[D->form] = K_ERROR;
        A.rerr[D->form] = E_TYPE;
        A.rword[D->form] = 0;
        continue;
      }
      V acc = mkv(A.H.tag[D->spine], A.H.word[D->spine]);
      for (uint32_t i = 1; i < D->nelem; ++i) fold_step(D->m, acc, mkv(A.H.tag[D->spine + i], A.H.word[D->spine + i]));
      A.rtag[D->form] = (uint8_t)acc.t;
      A.rword[D->form] = acc.w;
      continue;
    }
    if (!D->nonflat && A.payload) {
      // a flat list (no element is a cons): 2n+1 tokens written in parallel by culi_flat_export_kernel
      unsigned long long ntok = 2ull * D->n + 1;
      unsigned long long off = atomicAdd(A.pcount, ntok);
      if (off + ntok > A.pcap) {
        atomicExch(&A.flags[3], 1);
        A.rtag[D->form] = K_CONS;
        A.rword[D->form] = D->spine;
        continue;
      }
      A.desc[k].flat_off = off;
      A.rtag[D->form] = K_FLATREC;
      A.rword[D->form] = (off & 0xffffffffull) | (ntok << 32);
    } else {
      A.rtag[D->form] = K_CONS;
      A.rword[D->form] = D->spine;
    }
  }
}

// Export of flat ||| result lists (SURVEY §8(a)9 for the a6/a8 output): token 2i = the cons of cell i,
// token 2i+1 = element i, token 2n = nil.  Grid-stride over all elements of all flat descriptors.
__global__ void __launch_bounds__(256) culi_flat_export_kernel(const __grid_constant__ EvalArgs A) {
  uint32_t npend = *A.npend;
  if (npend > A.maxdesc) npend = A.maxdesc;
  uint32_t tid = blockIdx.x * blockDim.x + threadIdx.x, nth = gridDim.x * blockDim.x;
  for (uint32_t k = 0; k < npend; ++k) {
    const FanDesc* D = A.desc + k;
    if (A.rtag[D->form] != K_FLATREC) continue;
    uint32_t n = D->n, spine = D->spine;
    uint4* out = A.payload + D->flat_off;
    for (uint32_t i = tid; i < n; i += nth) {
      uint64_t cw = A.H.word[spine + i];
      uint32_t e = lo32(cw);
      uint32_t et = A.H.tag[e] & KIND_MASK;
      uint64_t ew = A.H.word[e];
      out[2 * i] = make_uint4(lo32(cw), hi32(cw), K_CONS, 0);
      out[2 * i + 1] = make_uint4(lo32(ew), hi32(ew), et, 0);
    }
    if (tid == 0) out[2 * n] = make_uint4(0, 0, K_NIL, 0);
  }
}

__global__ void culi_flat_commit_kernel(const __grid_constant__ EvalArgs A) {
  uint32_t npend = *A.npend;
  if (npend > A.maxdesc) npend = A.maxdesc;
  for (uint32_t k = threadIdx.x; k < npend; k += blockDim.x)
    if (A.rtag[A.desc[k].form] == K_FLATREC) A.rtag[A.desc[k].form] = K_CONS;
}

// ---- host launchers ----------------------------------------------------------------------------------
cudaError_t launch_relocate(cudaStream_t s, const uint8_t* stag, const uint64_t* sword, Node* nodes, uint64_t base,
                            uint64_t n, uint32_t str_base, uint32_t* roots, uint32_t nroots, int sms) {
  uint64_t work = n > nroots ? n : nroots;
  uint64_t blocks = (work + 255) / 256;
  if (blocks > (uint64_t)sms * 16) blocks = (uint64_t)sms * 16;
  if (blocks == 0) blocks = 1;
  culi_relocate_kernel<<<(unsigned)blocks, 256, 0, s>>>(stag, sword, nodes, base, n, str_base, roots, nroots);
  return cudaGetLastError();
}

size_t eval_smem_bytes(const EvalArgs& A) {
  return (size_t)A.code_n * sizeof(uint4) + (size_t)A.gst * 9 + 16;
}

cudaError_t launch_eval(cudaStream_t s, const EvalArgs& A, uint32_t blocks) {
  size_t smem = eval_smem_bytes(A);
  // specialised on whether the batch holds top-level ||| / wide forms (FANOUT), whether ||| can occur
  // below the top level (NEST) and whether idle warps split arguments off busy ones (SPLIT; not combined
  // with NEST, whose helpers use the idle warps)
  // and whether lane groups vote (VOTE: neither nesting nor splitting, code staging off)
  void (*k)(EvalArgs);
  if (A.nest) k = A.fanout ? culi_eval_kernel<true, true, false> : culi_eval_kernel<false, true, false>;
  else if (A.split) k = A.fanout ? culi_eval_kernel<true, false, true> : culi_eval_kernel<false, false, true>;
  else if (A.voting && A.code_n == 0) k = A.fanout ? culi_eval_vote_kernel<true> : culi_eval_vote_kernel<false>;
  else k = A.fanout ? culi_eval_kernel<true, false, false> : culi_eval_kernel<false, false, false>;
  if (smem > 48 * 1024) {
    cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
  }
  k<<<blocks, 128, smem, s>>>(A);
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

cudaError_t launch_reset(cudaStream_t s, unsigned long long* top, unsigned long long top_value,
                         uint32_t* next, unsigned long long* pcount, int* flags, uint32_t* npend,
                         uint32_t* nfallback, uint32_t* nnest, SplitCtl* sctl) {
  culi_reset_kernel<<<1, 1, 0, s>>>(top, top_value, next, pcount, flags, npend, nfallback, nnest, sctl);
  return cudaGetLastError();
}

cudaError_t launch_fanout(cudaStream_t s, const EvalArgs& A, uint32_t blocks) {
  size_t smem = eval_smem_bytes(A);
  if (smem > 48 * 1024) {
    cudaError_t e = cudaFuncSetAttribute(culi_fanout_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                         (int)smem);
    if (e != cudaSuccess) return e;
  }
  culi_fanout_kernel<<<blocks, 128, smem, s>>>(A);
  cudaError_t e = cudaGetLastError();
  if (e != cudaSuccess) return e;
  culi_fanout_finalize_kernel<<<1, 128, 0, s>>>(A);
  return cudaGetLastError();
}

cudaError_t launch_flat_export(cudaStream_t s, const EvalArgs& A, uint32_t blocks) {
  culi_flat_export_kernel<<<blocks, 256, 0, s>>>(A);
  cudaError_t e = cudaGetLastError();
  if (e != cudaSuccess) return e;
  culi_flat_commit_kernel<<<1, 128, 0, s>>>(A);
  return cudaGetLastError();
}

}  // namespace culi
