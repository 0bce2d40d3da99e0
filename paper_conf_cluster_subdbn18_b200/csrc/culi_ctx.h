// culi_ctx.h — session state of libculi.so (shared by culi_capi.cu and culi_dist.cu).
#pragma once
#include <cuda_runtime.h>

#include <algorithm>
#include <memory>
#include <string>
#include <vector>

#include "../../include/culi.h"
#include "culi_eval.cuh"
#include "culi_host.h"
#include "culi_reader.h"

inline uint32_t lo32h(uint64_t w) { return (uint32_t)w; }

using namespace culi;

struct culi_image {
  Image img;
  bool pinned = false;
  ~culi_image() {
    if (!pinned) return;
    if (!img.tag.empty()) cudaHostUnregister(img.tag.data());
    if (!img.word.empty()) cudaHostUnregister(img.word.data());
    if (!img.roots.empty()) cudaHostUnregister(img.roots.data());
  }
};

struct culi_results {
  Results r;
  bool ready = true;                 // false: an async batch's results before culi_sync
  struct culi_ctx* owner = nullptr;  // the ctx whose culi_sync completes them (while not ready)
};

namespace culi_detail {

template <typename T>
struct DevBuf {
  T* p = nullptr;
  size_t n = 0;
  cudaError_t ensure(size_t want) {
    if (want <= n) return cudaSuccess;
    if (p) cudaFree(p);
    p = nullptr;
    n = 0;
    size_t grow = std::max(want, (size_t)1024);
    cudaError_t e = cudaMalloc(&p, grow * sizeof(T));
    if (e == cudaSuccess) n = grow;
    return e;
  }
  void release() {
    if (p) cudaFree(p);
    p = nullptr;
    n = 0;
  }
};

constexpr uint32_t GCAP = 1u << 22;           // symbol ids supported (global table entries)
constexpr uint64_t STR_CAP = 64ull << 20;      // string bytes

// device reader working set (culi_reader.cu), allocated on first use
struct ReaderState {
  DevSyms S;
  uint32_t synced = 0;               // host names already in the device table
  uint64_t pool_top = 0;             // device name pool bytes mirrored on the host
  ReadInfo* info = nullptr;
  DevBuf<uint8_t> text, tiles, temp, ikind, ivt;
  DevBuf<uint32_t> tstate, toff, small, ipos, b32, roff, keys, keys2, vals, vals2, iparent, ij, ik, slen, soff, vlist;
  DevBuf<int> a32, depth, hmax;
  DevBuf<uint64_t> ival;
  float last_ms = 0;
  uint64_t last_items = 0, last_nodes = 0, last_bytes = 0;
  void release() {
    cudaFree(S.key); cudaFree(S.id); cudaFree(S.tag); cudaFree(S.noff); cudaFree(S.pool); cudaFree(S.count); cudaFree(info);
    S = DevSyms{};
    info = nullptr;
    for (auto* b : {&text, &tiles, &temp, &ikind, &ivt}) b->release();
    for (auto* b : {&tstate, &toff, &small, &ipos, &b32, &roff, &keys, &keys2, &vals, &vals2, &iparent, &ij, &ik,
                    &slen, &soff, &vlist})
      b->release();
    for (auto* b : {&a32, &depth, &hmax}) b->release();
    ival.release();
  }
};

// heap reclamation working set (culi_gc.cu)
struct GcState {
  DevBuf<uint32_t> role, pos, q0, q1, cnt;
  DevBuf<uint8_t> temp;
  uint32_t last_rounds = 0;
  uint64_t last_live = 0, last_freed = 0, total_freed = 0, collections = 0;
  void release() {
    for (auto* b : {&role, &pos, &q0, &q1, &cnt}) b->release();
    temp.release();
  }
};

}  // namespace culi_detail
using namespace culi_detail;

namespace culi {
int collect_persistent(culi_ctx* c, uint64_t* live, uint64_t* freed);
}

struct culi_ctx {
  culi_opts opts;
  cudaStream_t stream = nullptr;
  int sms = 0;
  bool arena_owned = true;           // heap / global frame / strings / stacks cudaMalloc'ed here (else opts.heap_base)
  culi_results* pending = nullptr;   // culi_eval_batch_async results awaiting culi_sync
  std::shared_ptr<SymTable> syms = std::make_shared<SymTable>();
  uint64_t str_cap = STR_CAP;
  std::string strings;              // host mirror of the device string area (persistent part)
  uint64_t mark = IMG_FIRST;        // first free heap node after the persistent (define) segment
  bool defined = false;
  // device memory
  DevHeap H{};
  uint4* kst = nullptr;
  uint4* vst = nullptr;
  uint32_t nslots = 0, kcap = 0, vcap = 0;
  uint32_t* next = nullptr;         // work counter
  unsigned long long* pcount = nullptr;
  int* flags = nullptr;             // [0] oom [1] define fail idx+1 [2] define err [3] payload ovf [4] export ovf
  DevBuf<uint32_t> roots, keys, keys_alt, perm, perm_alt;
  DevBuf<uint8_t> rtag, rerr, dtemp;
  DevBuf<uint64_t> stage;             // host image (SoA tag + word) before the relocate kernel interleaves it
  DevBuf<uint64_t> rsteps, rword;
  DevBuf<uint4> payload;
  // ||| fan-out state
  FanDesc* desc = nullptr;
  uint32_t maxdesc = 4096;
  uint32_t* npend = nullptr;
  uint32_t* nfallback = nullptr;
  DevBuf<uint32_t> fallback;
  bool batch_has_par = false;
  bool batch_has_wide = false;
  // nested ||| (§8(f)1)
  bool persist_has_par = false;      // some definition mentions |||
  bool persist_has_setq = false;     // some definition mentions setq (R7: batches run with heap frames)
  bool batch_mut = false, define_mut = false;
  bool persist_has_closure = false;  // some definition mentions lambda / defun
  bool batch_may_close = false;      // a closure may be applied in the batch (argument splitting useful)
  bool batch_single_par = false;     // the batch is one top-level (||| ...) form (its elements fan out)
  bool batch_may_nest = false;
  NestDesc* ndesc = nullptr;
  uint32_t maxnest = 4096;
  uint32_t* nnest = nullptr;         // [0] descriptors written, [1] forms finished
  uint4* kst2 = nullptr;             // secondary stacks, allocated on first use
  uint4* vst2 = nullptr;
  uint32_t last_fanout = 0, last_fallback = 0, last_nested = 0, last_splits = 0;
  // argument splitting
  SplitGroup* groups = nullptr;      // SPLIT_GPW per warp of the grid
  unsigned long long* gqueue = nullptr;
  uint32_t gqcap = 1u << 18;         // > outstanding tickets (<= warps of the grid + racing publishers)
  SplitCtl* sctl = nullptr;          // queue counters (persist across launches), tokens, stats, diagnostics
  unsigned long long wait_ns = 10ull * 1000 * 1000 * 1000;   // bounded inter-warp waits (env CULI_WAIT_MS)
  uint32_t last_timeouts = 0;
  uint32_t last_claimed = 0;         // split tasks a thief claimed in the last fetch
  uint32_t last_regrows = 0;         // payload-buffer regrowths (eval + export re-run) in the last fetch
  uint32_t last_diag[9] = {0};
  uint32_t split_poll = 64;          // closure calls between polls (env CULI_SPLIT_POLL)
  uint32_t split_first = 64;         // closure calls before the first poll (env CULI_SPLIT_FIRST)
  uint32_t steal_gate = 1;           // steal only from fully idle warps (env CULI_STEAL_GATE)
  uint32_t split_sleep = 4096;       // idle-warp back-off cap in ns (env CULI_SPLIT_SLEEP)
  uint32_t size_first = 1;           // dispatch: closure-free batches biggest forms first (env CULI_SIZE_FIRST)
  bool force_device_read = false;    // env CULI_DEVICE_READ=1: culi_*_text never uses the host reader
  uint32_t thin_lanes = 0;           // small plain-kernel batches: forms per warp (0 = auto; env CULI_THIN_LANES)
  DevBuf<uint32_t> wide;
  DevBuf<uint32_t> lenpairs;         // wide-list length marks of a host image (culi_lenmark_kernel)
  // uploaded batch (culi_upload)
  bool have_batch = false;
  uint64_t batch_nodes = 0;
  uint32_t batch_forms = 0;
  uint32_t* batch_perm = nullptr;
  std::string batch_strings;
  ReaderState rd;
  GcState gc;
  cudaGraphExec_t graph_exec = nullptr;  // culi_eval_uploaded replay of the uploaded batch
  uint32_t graph_kernels = 0;
  // timing
  cudaEvent_t ev[4] = {nullptr, nullptr, nullptr, nullptr};
  uint32_t last_kernels = 0;
  uint64_t heap_high = 0;
};

