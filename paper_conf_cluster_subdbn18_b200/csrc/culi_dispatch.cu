// culi_dispatch.cu — classify + bin the forms of a batch before evaluation.
//
// The paper notes that divergent branches of a warp are serialised (§III-D.d).  Forms are
// independent, so their evaluation order is free: we give each form a 64-bit key
//   (30-bit structure prefix << 26) | (10-bit shape hash << 16) | (0xffff - cost hint)
// where the structure prefix is the form's first five pre-order tokens (list open, number kinds, a
// user-symbol bucket before the reserved operators — user functions are the heavy forms, so they start
// first; 6 bits each, most significant first, so forms that share
// a beginning sort next to each other even when they differ later), the shape hash covers the form's
// first 48 nodes (kinds, symbols, structure; not number values) so identical shapes are contiguous inside
// a prefix, and the cost hint is the first argument when it is an integer literal (e.g. n of (fib n)), so
// forms whose control flow is identical land in the same warp, heaviest first.  (C4: 114,763 distinct
// shapes among 262,144 forms, two thirds of the forms in shape classes smaller than a warp — the prefix
// keeps near-identical ones together.)  A radix sort (CUB, a plain library sort) of (key, form) gives the
// evaluation permutation; consecutive forms of it go to the lanes of a warp.
#include <cub/device/device_radix_sort.cuh>
#include <cuda_runtime.h>

#include "culi_eval.cuh"

namespace culi {

// Shape of a form: FNV-1a over a pre-order walk of its first 48 nodes — node kinds, symbol ids, list
// structure; numbers contribute only their kind (their values are in the hint).  Forms with equal shape
// expand macros and take calls in the same order, so a warp of them stays converged longer (C4).
// *size: nodes visited (at most 48) — a cost proxy for batches without closures, where a form's work is
// bounded by its size (no recursion): their warps run the biggest forms first (longest processing time
// first), so the last, partly filled round of warp batches holds small ones.
__device__ uint32_t shape_hash(TagArr tag, WordArr word, uint32_t x, uint32_t* size) {
  uint32_t st[12];
  int sp = 0;
  uint32_t h = 2166136261u;
  int visited = 0;
  for (; visited < 48; ++visited) {
    uint32_t t = tag[x] & KIND_MASK;
    h = (h ^ t) * 16777619u;
    if (t == K_SYM) h = (h ^ (uint32_t)word[x]) * 16777619u;
    if (t == K_CONS) {
      uint64_t w = word[x];
      uint32_t cdr = (uint32_t)(w >> 32);
      if (cdr) {
        if (sp < 12) st[sp++] = cdr;
        else h = (h ^ 0x9e3779b9u) * 16777619u;
      }
      x = (uint32_t)w;
      continue;
    }
    if (sp == 0) break;
    x = st[--sp];
    h = (h ^ 0x55u) * 16777619u;                      // a subtree ended: keeps (a (b) c) != (a (b c))
  }
  *size = (uint32_t)visited + 1;
  return h;
}

static_assert(16 + N_RESERVED <= 64, "reserved-operator token codes fit in 6 bits");
// Pre-order token stream of a form, most significant first: 6 bits per token, the first five tokens.
__device__ uint64_t structure_prefix(TagArr tag, WordArr word, uint32_t x) {
  uint32_t st[8];
  int sp = 0, n = 0;
  uint64_t key = 0;
  auto emit = [&](uint32_t code) {
    if (n < 5) key |= (uint64_t)(code & 63u) << (6 * (4 - n));
    ++n;
  };
  for (int visited = 0; visited < 24 && n < 5; ++visited) {
    uint32_t t = tag[x] & KIND_MASK;
    if (t == K_CONS) {
      uint64_t w = word[x];
      uint32_t cdr = (uint32_t)(w >> 32);
      emit(1);                                           // a list opens (its elements follow)
      if (cdr && sp < 8) st[sp++] = cdr;
      x = (uint32_t)w;
      continue;
    }
    uint32_t code = t == K_INT ? 3 : t == K_FLOAT ? 4 : t == K_STR ? 5 : t == K_NIL ? 6 : t == K_T ? 7 : 2;
    if (t == K_SYM) {
      uint32_t sid = (uint32_t)word[x];
      code = sid < N_RESERVED ? 16 + sid : 8 + (sid & 7u);    // user functions first: heaviest work early
    }
    emit(code);
    if (sp == 0) break;
    x = st[--sp];
  }
  return key;
}

__global__ void culi_classify_kernel(TagArr tag, WordArr word,
                                     const uint32_t* __restrict__ roots, uint32_t nforms,
                                     unsigned long long* __restrict__ keys, uint32_t* __restrict__ perm,
                                     uint32_t size_first) {
  uint32_t stride = gridDim.x * blockDim.x;
  for (uint32_t f = blockIdx.x * blockDim.x + threadIdx.x; f < nforms; f += stride) {
    uint32_t r = roots[f];
    uint32_t hint = 0, shape = 0, size = 1;
    uint64_t prefix = structure_prefix(tag, word, r);
    if ((tag[r] & KIND_MASK) == K_CONS) {
      uint64_t w = word[r];
      uint32_t rest = (uint32_t)(w >> 32);
      if (rest != 0) {
        uint32_t a = (uint32_t)word[rest];
        uint32_t at = tag[a] & KIND_MASK;
        if (at == K_INT) {
          long long v = (long long)word[a];
          hint = v < 0 ? 0 : (v > 0xffff ? 0xffff : (uint32_t)v);
        } else if (at == K_CONS) {
          uint32_t ah = (uint32_t)word[a];                // head symbol of a nested first argument
          if ((tag[ah] & KIND_MASK) == K_SYM) hint = 0xff00u | ((uint32_t)word[ah] & 0xff);
        }
      }
      shape = shape_hash(tag, word, r, &size);
    }
    // 56 bits (7 radix passes): structure prefix 30 | shape hash 10 | inverted hint 16; closure-free batches:
    // inverted size class 4 (nodes / 4, up to 48 nodes) | structure prefix 30 | shape hash 10 | inverted hint 12
    uint64_t sh = (uint64_t)((shape ^ (shape >> 10) ^ (shape >> 20)) & 0x3ffu);
    if (size_first) {
      uint32_t cls = min(size / 4u, 15u);
      keys[f] = ((uint64_t)(15u - cls) << 52) | (prefix << 22) | (sh << 12) | (0xfffu - min(hint, 0xfffu));
    } else {
      keys[f] = (prefix << 26) | (sh << 16) | (0xffffu - hint);
    }
    perm[f] = f;
  }
}

// classify + CUB histogram + exclusive sum + 7 one-sweep passes (56 key bits)
uint32_t dispatch_launches(uint32_t) { return 10u; }

size_t dispatch_temp_bytes(uint32_t nforms) {
  size_t bytes = 0;
  cub::DeviceRadixSort::SortPairs((void*)nullptr, bytes, (const unsigned long long*)nullptr,
                                  (unsigned long long*)nullptr, (const uint32_t*)nullptr, (uint32_t*)nullptr,
                                  (int)nforms);
  return bytes + 256;
}

cudaError_t launch_dispatch(cudaStream_t s, const DevHeap& H, const uint32_t* roots, uint32_t nforms,
                            uint32_t* keys, uint32_t* keys_alt, uint32_t* perm, uint32_t* perm_alt,
                            void* temp, size_t temp_bytes, uint32_t** perm_out, int sms, uint32_t size_first) {
  // keys / keys_alt hold 2 x nforms words each (64-bit keys)
  unsigned long long* k0 = reinterpret_cast<unsigned long long*>(keys);
  unsigned long long* k1 = reinterpret_cast<unsigned long long*>(keys_alt);
  uint32_t blocks = (nforms + 255) / 256;
  if (blocks > (uint32_t)sms * 8) blocks = sms * 8;
  if (blocks == 0) blocks = 1;
  culi_classify_kernel<<<blocks, 256, 0, s>>>(H.tag, H.word, roots, nforms, k0, perm, size_first);
  cudaError_t e = cudaGetLastError();
  if (e != cudaSuccess) return e;
  size_t tb = temp_bytes;
  e = cub::DeviceRadixSort::SortPairs(temp, tb, k0, k1, perm, perm_alt, (int)nforms, 0, 56, s);
  *perm_out = perm_alt;
  return e;
}

}  // namespace culi
