// culi_gc.cu — heap reclamation of the persistent segment.
//
// The paper allocates "the sequentially next free node" of a fixed node array and marks nodes that are no
// longer needed as free (§III-A.c).  Here batch allocations are already released wholesale
// (the bump pointer returns to the post-define mark after every batch); what grows over a long session is
// the persistent segment [IMG_FIRST, mark): definition images and the temporaries their evaluation made.
// After culi_define this pass keeps exactly the nodes reachable from the global frame and slides them
// down in address order (mark-compact):
//   mark    — parallel graph traversal from the global table, in rounds over a frontier of structural
//             objects (cons runs, closures, frames).  A cons cell is taken with its whole contiguous run
//             (cdr == next cell), 32 cells per warp step, so a 1M-element reader list is one object, not a
//             1M-long pointer chain.  Every node is claimed once (atomicCAS on its role), leaves are never
//             queued.  Roles record how a node's word is remapped (closure AUX nodes, frame value slots).
//   compact — exclusive scan of the live flags gives each live node its new index; nodes are copied,
//             references remapped, into scratch space above the mark, then back; global values remapped.
// Sliding preserves the relative order of live nodes, so a list spine that was contiguous stays
// contiguous (SURVEY c.14: ||| keeps its O(1) element indexing), node identity is a bijection (eq),
// and everything else (tags, TAG_VALID, string offsets, symbol ids) is copied verbatim.
#include <cub/device/device_scan.cuh>
#include <cuda_runtime.h>

#include "culi_ctx.h"

namespace culi {
namespace gc {

enum : uint32_t { R_DEAD = 0, R_NODE = 1, R_RAW = 2, R_AUX2 = 3 };
constexpr uint32_t REFS = (1u << K_STR) | (1u << K_CONS) | (1u << K_CLOSURE) | (1u << K_MACRO);
constexpr uint32_t STRUCT = (1u << K_CONS) | (1u << K_CLOSURE) | (1u << K_MACRO) | (1u << K_FRAME);

struct Args {
  TagArr tag;                   // views of the heap's node array
  WordArr word;
  uint64_t mark;
  uint32_t* role;               // per node of [0, mark)
  const uint32_t* in;           // frontier of this round
  uint32_t* out;                // frontier of the next round
  uint32_t* cnt;                // [0] items in `in`, [1] next item to take, [2] items in `out`
};

__device__ __forceinline__ uint32_t lo(uint64_t w) { return (uint32_t)w; }
__device__ __forceinline__ uint32_t hi(uint64_t w) { return (uint32_t)(w >> 32); }

// a reference found in a live node: claim it; queue it when it has references of its own
__device__ __forceinline__ void visit(const Args& G, uint32_t y) {
  if (y < IMG_FIRST || y >= G.mark) return;
  if (atomicCAS(G.role + y, R_DEAD, R_NODE) != R_DEAD) return;
  if ((STRUCT >> (G.tag[y] & KIND_MASK)) & 1u) G.out[atomicAdd(G.cnt + 2, 1u)] = y;
}

__global__ void roots_kernel(Args G, const uint8_t* gtag, const uint64_t* gword, uint32_t nsyms) {
  for (uint32_t s = blockIdx.x * blockDim.x + threadIdx.x; s < nsyms; s += gridDim.x * blockDim.x)
    if ((REFS >> (gtag[s] & KIND_MASK)) & 1u) visit(G, (uint32_t)gword[s]);
}

// one warp per queued object
__global__ void trace_kernel(Args G) {
  const int lane = threadIdx.x & 31;
  for (;;) {
    uint32_t it = 0;
    if (lane == 0) it = atomicAdd(G.cnt + 1, 1u);
    it = __shfl_sync(0xffffffffu, it, 0);
    if (it >= G.cnt[0]) return;
    uint32_t x = G.in[it];
    uint32_t k = G.tag[x] & KIND_MASK;
    if (k == K_CONS) {
      // the run of consecutive cells starting at x (x itself was claimed by whoever queued it)
      for (uint64_t base = x;; base += 32) {
        uint64_t c = base + lane;
        bool in = c < G.mark;
        uint32_t t = in ? (G.tag[c] & KIND_MASK) : 0;
        uint64_t w = in ? G.word[c] : 0;
        bool cons = t == K_CONS;
        bool next_cons = __shfl_down_sync(0xffffffffu, cons, 1);
        if (lane == 31) next_cons = c + 1 < G.mark && (G.tag[c + 1] & KIND_MASK) == K_CONS;
        bool link = cons && hi(w) == c + 1 && next_cons;
        unsigned brk = __ballot_sync(0xffffffffu, !link);
        int last = brk ? __ffs(brk) - 1 : 31;           // last run cell in this chunk
        bool mine = false;
        if (lane <= last) mine = (c == x) || atomicCAS(G.role + c, R_DEAD, R_NODE) == R_DEAD;
        if (mine) {
          visit(G, lo(w));
          if (lane == last && brk) visit(G, hi(w));     // the run's end: its cdr leaves the run
        }
        unsigned lost = __ballot_sync(0xffffffffu, lane <= last && !mine);
        if (brk || lost) break;                         // run ended, or the rest belongs to another tracer
      }
    } else if (k == K_CLOSURE || k == K_MACRO) {        // {code | env} {AUX np | first} {AUX body | params}
      if (lane == 0) {
        uint64_t w = G.word[x], a2 = G.word[x + 2];
        G.role[x + 1] = R_RAW;
        G.role[x + 2] = R_AUX2;
        visit(G, lo(w));
        visit(G, hi(w));
        visit(G, lo(a2));
        visit(G, hi(a2));
      }
    } else if (k == K_FRAME) {                          // {parent | n} n x {BIND sym | value node} n slots
      uint64_t w = G.word[x];
      uint32_t n = hi(w);
      if (lane == 0) visit(G, lo(w));
      for (uint32_t i = lane; i < n; i += 32) {
        G.role[x + 1 + i] = R_NODE;
        visit(G, hi(G.word[x + 1 + i]));
      }
    }
  }
}

__global__ void live_kernel(const uint32_t* role, uint64_t mark, uint32_t* live) {
  for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < mark; i += (uint64_t)gridDim.x * blockDim.x)
    live[i] = (i >= IMG_FIRST && role[i] != R_DEAD) ? 1u : 0u;
}

__device__ __forceinline__ uint32_t fwd(const uint32_t* pos, uint32_t y) {
  return y < IMG_FIRST ? y : IMG_FIRST + pos[y];
}

// live node i -> scratch[pos[i]], references remapped
__global__ void copy_kernel(TagArr tag, WordArr word, const uint32_t* role, const uint32_t* pos,
                            uint64_t mark, TagArr stag, WordArr sword) {
  for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < mark; i += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t r = role[i];
    if (i < IMG_FIRST || r == R_DEAD) continue;
    const uint4 q = *reinterpret_cast<const uint4*>(tag.p + i);     // the whole node (incl. a TAG_LEN length)
    uint8_t t = (uint8_t)q.z;
    uint64_t w = ((uint64_t)q.y << 32) | q.x;
    if (r == R_AUX2) {
      w = pack2(fwd(pos, lo(w)), fwd(pos, hi(w)));
    } else if (r == R_NODE) {
      switch (t & KIND_MASK) {
        case K_CONS: w = pack2(fwd(pos, lo(w)), fwd(pos, hi(w))); break;
        case K_CLOSURE:
        case K_MACRO: w = pack2(fwd(pos, lo(w)), fwd(pos, hi(w))); break;
        case K_FRAME: w = pack2(fwd(pos, lo(w)), hi(w)); break;
        case K_BIND: w = pack2(lo(w), fwd(pos, hi(w))); break;
        default: break;                                 // leaves: payload verbatim
      }
    }
    uint32_t d = pos[i];                              // (compaction keeps spines contiguous: lengths stay valid)
    *reinterpret_cast<uint4*>(stag.p + d) = make_uint4((uint32_t)w, (uint32_t)(w >> 32), q.z, q.w);
    (void)sword;
  }
}

__global__ void globals_kernel(const uint8_t* gtag, uint64_t* gword, uint32_t nsyms, const uint32_t* pos) {
  for (uint32_t s = blockIdx.x * blockDim.x + threadIdx.x; s < nsyms; s += gridDim.x * blockDim.x)
    if ((REFS >> (gtag[s] & KIND_MASK)) & 1u) gword[s] = fwd(pos, (uint32_t)gword[s]);
}

}  // namespace gc

#define GK(x)                                  \
  do {                                         \
    cudaError_t e_ = (x);                      \
    if (e_ != cudaSuccess) return CULI_E_CUDA; \
  } while (0)

// Compact the persistent segment; *live / *freed in nodes (of [IMG_FIRST, mark)).  A segment that has no
// scratch room above it (mark + live > capacity) is left as it is.
int collect_persistent(culi_ctx* c, uint64_t* live_out, uint64_t* freed_out) {
  using namespace gc;
  uint64_t mark = c->mark;
  if (live_out) *live_out = mark - IMG_FIRST;
  if (freed_out) *freed_out = 0;
  if (mark <= IMG_FIRST) return CULI_OK;
  cudaStream_t st = c->stream;
  GcState& S = c->gc;
  GK(S.role.ensure(mark));
  GK(S.pos.ensure(mark + 1));
  GK(S.q0.ensure(mark));
  GK(S.q1.ensure(mark));
  GK(S.cnt.ensure(4));
  GK(cudaMemsetAsync(S.role.p, 0, mark * 4, st));
  GK(cudaMemsetAsync(S.cnt.p, 0, 16, st));
  uint32_t nsyms = (uint32_t)std::min<size_t>(c->syms->names.size(), c->H.gcap);
  Args G{c->H.tag, c->H.word, mark, S.role.p, S.q1.p, S.q0.p, S.cnt.p};
  unsigned blocks = (unsigned)c->sms * 8;
  roots_kernel<<<blocks, 256, 0, st>>>(G, c->H.gtag, c->H.gword, nsyms);
  GK(cudaGetLastError());
  uint32_t* qa = S.q0.p;
  uint32_t* qb = S.q1.p;
  for (uint32_t round = 0;; ++round) {
    uint32_t n = 0;
    GK(cudaMemcpyAsync(&n, S.cnt.p + 2, 4, cudaMemcpyDeviceToHost, st));
    GK(cudaStreamSynchronize(st));
    if (n == 0) break;
    uint32_t cnt[3] = {n, 0, 0};
    GK(cudaMemcpyAsync(S.cnt.p, cnt, 12, cudaMemcpyHostToDevice, st));
    G.in = qa;
    G.out = qb;
    unsigned warps = std::min<uint32_t>(n, (uint32_t)c->sms * 64);
    trace_kernel<<<(warps + 7) / 8, 256, 0, st>>>(G);
    GK(cudaGetLastError());
    std::swap(qa, qb);
    S.last_rounds = round + 1;
  }
  // live flags -> new positions
  live_kernel<<<blocks, 256, 0, st>>>(S.role.p, mark, S.pos.p);
  GK(cudaMemsetAsync(S.pos.p + mark, 0, 4, st));
  size_t tb = 0;
  GK(cub::DeviceScan::ExclusiveSum(nullptr, tb, S.pos.p, S.pos.p, (int)(mark + 1), st));
  GK(S.temp.ensure(tb + 16));
  GK(cub::DeviceScan::ExclusiveSum(S.temp.p, tb, S.pos.p, S.pos.p, (int)(mark + 1), st));
  uint32_t live = 0;
  GK(cudaMemcpyAsync(&live, S.pos.p + mark, 4, cudaMemcpyDeviceToHost, st));
  GK(cudaStreamSynchronize(st));
  if (live_out) *live_out = live;
  if (mark + live > c->H.cap) return CULI_OK;           // no scratch room: keep the segment as it is
  copy_kernel<<<blocks, 256, 0, st>>>(c->H.tag, c->H.word, S.role.p, S.pos.p, mark, c->H.tag + mark, c->H.word + mark);
  GK(cudaGetLastError());
  if (live)
    GK(cudaMemcpyAsync(c->H.tag.p + IMG_FIRST, c->H.tag.p + mark, (size_t)live * sizeof(Node), cudaMemcpyDeviceToDevice, st));
  globals_kernel<<<blocks, 256, 0, st>>>(c->H.gtag, c->H.gword, nsyms, S.pos.p);
  GK(cudaGetLastError());
  GK(cudaStreamSynchronize(st));
  if (freed_out) *freed_out = mark - IMG_FIRST - live;
  c->mark = IMG_FIRST + live;
  return CULI_OK;
}

}  // namespace culi
