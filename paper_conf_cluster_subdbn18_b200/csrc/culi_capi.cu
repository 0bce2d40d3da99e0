// culi_capi.cu — the C-ABI of libculi.so (include/culi.h): session state, device memory, uploads,
// kernel launches and result copies.  No CPU fallback: every step of eval runs in the kernels of
// culi_kernels.cu / culi_dispatch.cu.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <memory>
#include <new>
#include <string>
#include <vector>

#include "../../include/culi.h"
#include "culi_eval.cuh"
#include "culi_host.h"
#include "culi_ctx.h"



using namespace culi;

#define CK(x)                                   \
  do {                                          \
    cudaError_t _e = (x);                       \
    if (_e != cudaSuccess) return CULI_E_CUDA;  \
  } while (0)

static void drop_graph(culi_ctx* c) {
  if (c->graph_exec) cudaGraphExecDestroy(c->graph_exec);
  c->graph_exec = nullptr;
}

// Caller-owned arena (culi_opts.heap_base): heap nodes (16 B each), global frame tag + word, string area,
// K- and V-stacks, each 256-byte aligned, in this order.
struct ArenaLayout {
  size_t off[6];
  size_t total;
};
static ArenaLayout arena_layout(uint64_t heap_nodes, uint64_t str_cap, size_t nslots, size_t kcap, size_t vcap) {
  size_t sz[6] = {heap_nodes * sizeof(Node), GCAP, (size_t)GCAP * 8, str_cap, nslots * kcap * 16, nslots * vcap * 16};
  ArenaLayout L{};
  size_t o = 0;
  for (int k = 0; k < 6; ++k) {
    L.off[k] = o;
    o = (o + sz[k] + 255) & ~(size_t)255;
  }
  L.total = o;
  return L;
}

// opts with defaults filled in; false on an invalid value
static bool normalize_opts(culi_opts& o, int sms) {
  if (o.max_depth == 0) o.max_depth = 1024;
  if (o.max_depth > 4095) return false;
  if (o.fuel == 0) o.fuel = 1ull << 40;
  if (o.heap_nodes == 0) o.heap_nodes = 64ull << 20;
  if (o.heap_nodes > 0x7fffffffull) return false;
  if (o.vstack_entries == 0) o.vstack_entries = 4096;
  if (o.vstack_entries > 65535) return false;
  if (o.slots == 0) o.slots = (uint32_t)sms * 128 * std::max(CULI_BLOCKS_PER_SM, CULI_SPLIT_BLOCKS_PER_SM);
  return true;
}

extern "C" {

int culi_arena_bytes(const culi_opts* opts, uint64_t* bytes) {
  if (!opts || !bytes) return CULI_E_ARG;
  culi_opts o = *opts;
  int ndev = 0, sms = 0;
  if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev <= 0 || o.device >= ndev) return CULI_E_CUDA;
  if (cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, o.device) != cudaSuccess) return CULI_E_CUDA;
  if (!normalize_opts(o, sms)) return CULI_E_ARG;
  size_t nslots = (o.slots + 127) / 128 * 128;
  *bytes = arena_layout(o.heap_nodes, STR_CAP, nslots, 2 * o.max_depth + 8, o.vstack_entries).total;
  return CULI_OK;
}

void culi_default_opts(culi_opts* o) {
  if (!o) return;
  std::memset(o, 0, sizeof *o);
}

const char* culi_status_string(int s) {
  switch (s) {
    case CULI_OK: return "ok";
    case CULI_E_ARG: return "bad argument";
    case CULI_E_PARSE: return "parse error";
    case CULI_E_HEAP_FULL: return "device heap or stack exhausted";
    case CULI_E_CUDA: return "CUDA error";
    case CULI_E_NCCL: return "NCCL error";
    case CULI_E_DEFINE: return "definition failed";
    case CULI_E_STATE: return "invalid state";
  }
  return "unknown status";
}

const char* culi_error_name(uint8_t e) { return e < 10 ? kErrName[e] : "?"; }

int culi_init(const culi_opts* opts, culi_ctx** out) {
  if (!out) return CULI_E_ARG;
  *out = nullptr;
  culi_ctx* c = new (std::nothrow) culi_ctx;
  if (!c) return CULI_E_ARG;
  culi_default_opts(&c->opts);
  if (opts) c->opts = *opts;
  culi_opts& o = c->opts;
  int ndev = 0;
  if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev <= 0 || o.device >= ndev) {
    delete c;
    return CULI_E_CUDA;
  }
  if (cudaSetDevice(o.device) != cudaSuccess) { delete c; return CULI_E_CUDA; }
  cudaDeviceGetAttribute(&c->sms, cudaDevAttrMultiProcessorCount, o.device);
  if (!normalize_opts(o, c->sms)) { delete c; return CULI_E_ARG; }
  c->nslots = (o.slots + 127) / 128 * 128;
  c->kcap = 2 * o.max_depth + 8;
  c->vcap = o.vstack_entries;
  c->stream = (cudaStream_t)o.stream;
  if (const char* e = getenv("CULI_SPLIT_POLL")) c->split_poll = std::max(1, atoi(e));      // tuning knobs
  if (const char* e = getenv("CULI_SPLIT_FIRST")) c->split_first = std::max(1, atoi(e));
  if (const char* e = getenv("CULI_SPLIT_SLEEP")) c->split_sleep = std::max(32, atoi(e));
  if (const char* e = getenv("CULI_STEAL_GATE")) c->steal_gate = atoi(e) != 0;
  if (const char* e = getenv("CULI_SIZE_FIRST")) c->size_first = atoi(e) != 0;
  if (const char* e = getenv("CULI_DEVICE_READ")) c->force_device_read = atoi(e) != 0;
  if (const char* e = getenv("CULI_THIN_LANES")) c->thin_lanes = std::min(32, std::max(0, atoi(e)));
  if (const char* e = getenv("CULI_WAIT_MS")) c->wait_ns = (unsigned long long)std::max(1, atoi(e)) * 1000000ull;
  bool ok = true;
  if (o.heap_base) {                                 // caller-owned arena (e.g. a torch tensor)
    ArenaLayout L = arena_layout(o.heap_nodes, c->str_cap, c->nslots, c->kcap, c->vcap);
    if (o.heap_bytes < L.total || ((uintptr_t)o.heap_base & 255)) { delete c; return CULI_E_ARG; }
    char* b = (char*)o.heap_base;
    c->arena_owned = false;
    c->H.tag = TagArr{(Node*)(b + L.off[0])};
    c->H.word = WordArr{c->H.tag.p};
    c->H.gtag = (uint8_t*)(b + L.off[1]);
    c->H.gword = (uint64_t*)(b + L.off[2]);
    c->H.strs = (const char*)(b + L.off[3]);
    c->kst = (uint4*)(b + L.off[4]);
    c->vst = (uint4*)(b + L.off[5]);
  } else {
    Node* nodes = nullptr;
    ok &= cudaMalloc(&nodes, o.heap_nodes * sizeof(Node)) == cudaSuccess;
    c->H.tag = TagArr{nodes};
    c->H.word = WordArr{nodes};
    ok &= cudaMalloc(&c->H.gtag, GCAP) == cudaSuccess;
    ok &= cudaMalloc(&c->H.gword, (size_t)GCAP * 8) == cudaSuccess;
    ok &= cudaMalloc((void**)&c->H.strs, c->str_cap) == cudaSuccess;
    ok &= cudaMalloc(&c->kst, (size_t)c->nslots * c->kcap * sizeof(uint4)) == cudaSuccess;
    ok &= cudaMalloc(&c->vst, (size_t)c->nslots * c->vcap * sizeof(uint4)) == cudaSuccess;
  }
  ok &= cudaMalloc(&c->H.top, sizeof(unsigned long long)) == cudaSuccess;
  ok &= cudaMalloc(&c->next, sizeof(uint32_t)) == cudaSuccess;
  ok &= cudaMalloc(&c->pcount, sizeof(unsigned long long)) == cudaSuccess;
  ok &= cudaMalloc(&c->flags, 8 * sizeof(int)) == cudaSuccess;
  ok &= cudaMalloc(&c->desc, (size_t)c->maxdesc * sizeof(FanDesc)) == cudaSuccess;
  ok &= cudaMalloc(&c->npend, sizeof(uint32_t)) == cudaSuccess;
  ok &= cudaMalloc(&c->nfallback, sizeof(uint32_t)) == cudaSuccess;
  ok &= cudaMalloc(&c->nnest, 2 * sizeof(uint32_t)) == cudaSuccess;
  ok &= cudaMalloc(&c->ndesc, (size_t)c->maxnest * sizeof(NestDesc)) == cudaSuccess;
  ok &= cudaMalloc(&c->groups, (size_t)c->nslots / 32 * SPLIT_GPW * sizeof(SplitGroup)) == cudaSuccess;
  ok &= cudaMalloc(&c->gqueue, (size_t)c->gqcap * sizeof(unsigned long long)) == cudaSuccess;
  ok &= cudaMalloc(&c->sctl, sizeof(SplitCtl)) == cudaSuccess;
  for (int k = 0; k < 4 && ok; ++k) ok &= cudaEventCreate(&c->ev[k]) == cudaSuccess;
  if (!ok) { culi_shutdown(c); return CULI_E_CUDA; }
  c->H.cap = o.heap_nodes;
  c->H.gcap = GCAP;
  // nil and T nodes; every symbol unbound; builtins are resolved by id (reserved names)
  static const Node n01[2] = {Node{0, K_NIL, {}, 0}, Node{0, K_T, {}, 0}};
  bool ok2 = cudaMemcpyAsync(c->H.tag.p, n01, sizeof(n01), cudaMemcpyHostToDevice, c->stream) == cudaSuccess &&
             cudaMemsetAsync(c->H.gtag, K_UNBOUND, GCAP, c->stream) == cudaSuccess &&
             cudaMemsetAsync(c->flags, 0, 8 * sizeof(int), c->stream) == cudaSuccess &&
             cudaMemsetAsync(c->groups, 0xff, (size_t)c->nslots / 32 * SPLIT_GPW * sizeof(SplitGroup), c->stream) == cudaSuccess &&
             cudaMemsetAsync(c->gqueue, 0, (size_t)c->gqcap * sizeof(unsigned long long), c->stream) == cudaSuccess &&
             cudaMemsetAsync(c->sctl, 0, sizeof(SplitCtl), c->stream) == cudaSuccess &&
             cudaStreamSynchronize(c->stream) == cudaSuccess;
  if (!ok2) { culi_shutdown(c); return CULI_E_CUDA; }
  *out = c;
  return CULI_OK;
}

void culi_shutdown(culi_ctx* c) {
  if (!c) return;
  cudaStreamSynchronize(c->stream);
  if (c->pending) {                                  // an async batch nobody synced: results stay not ready
    c->pending->owner = nullptr;
    c->pending = nullptr;
  }
  if (c->arena_owned) {
    cudaFree(c->H.tag.p);
    cudaFree(c->H.gtag);
    cudaFree(c->H.gword);
    cudaFree((void*)c->H.strs);
    cudaFree(c->kst);
    cudaFree(c->vst);
  }
  cudaFree(c->H.top);
  cudaFree(c->next);
  cudaFree(c->pcount);
  cudaFree(c->flags);
  cudaFree(c->desc);
  cudaFree(c->npend);
  cudaFree(c->nfallback);
  cudaFree(c->nnest);
  cudaFree(c->ndesc);
  cudaFree(c->groups);
  cudaFree(c->gqueue);
  cudaFree(c->sctl);
  cudaFree(c->kst2);
  cudaFree(c->vst2);
  c->fallback.release();
  c->wide.release();
  c->roots.release(); c->keys.release(); c->keys_alt.release(); c->perm.release();
  c->perm_alt.release(); c->rtag.release(); c->rerr.release(); c->dtemp.release();
  c->rsteps.release(); c->rword.release(); c->payload.release();
  drop_graph(c);
  c->rd.release();
  c->gc.release();
  for (auto& e : c->ev) if (e) cudaEventDestroy(e);
  delete c;
}

int culi_read(culi_ctx* c, const char* text, size_t len, culi_image** out, size_t* err_offset) {
  if (!c || !out || (!text && len)) return CULI_E_ARG;
  *out = nullptr;
  culi_image* im = new (std::nothrow) culi_image;
  if (!im) return CULI_E_ARG;
  int rc = read_image(*c->syms, text, len, im->img, err_offset);
  if (rc != CULI_OK) { delete im; return rc; }
  *out = im;
  return CULI_OK;
}

uint32_t culi_image_nforms(const culi_image* im) { return im ? (uint32_t)im->img.roots.size() : 0; }
uint64_t culi_image_nnodes(const culi_image* im) { return im ? im->img.tag.size() : 0; }
void culi_image_free(culi_image* im) { delete im; }

int culi_image_pin(culi_image* im, uint64_t* h2d_bytes) {
  if (!im) return CULI_E_ARG;
  const Image& g = im->img;
  if (h2d_bytes) *h2d_bytes = g.tag.size() * 9 + g.roots.size() * 4 + g.strings.size();
  if (im->pinned) return CULI_OK;
  bool ok = true;
  if (!g.tag.empty())
    ok &= cudaHostRegister((void*)g.tag.data(), g.tag.size(), cudaHostRegisterDefault) == cudaSuccess;
  if (!g.word.empty())
    ok &= cudaHostRegister((void*)g.word.data(), g.word.size() * 8, cudaHostRegisterDefault) == cudaSuccess;
  if (!g.roots.empty())
    ok &= cudaHostRegister((void*)g.roots.data(), g.roots.size() * 4, cudaHostRegisterDefault) == cudaSuccess;
  im->pinned = true;                                 // partial registrations are undone by the destructor
  return ok ? CULI_OK : CULI_E_CUDA;
}

}  // extern "C"

// ---- internal helpers ------------------------------------------------------------------------------
// Does the ||| symbol occur in the image?  With skip_root_heads, occurrences that are the head of a
// top-level form do not count: those forms go to the top-level fan-out (a6), never through nesting.
// (Symbol nodes are shared within an image, so look at the cons cells that refer to it.)
static bool image_mentions_par(const Image& img, bool skip_root_heads = false) {
  uint32_t par = 0;
  for (size_t k = 0; k < img.tag.size() && !par; ++k)
    if ((img.tag[k] & KIND_MASK) == K_SYM && img.word[k] == N_SPECIALS + BI_PAR) par = IMG_FIRST + (uint32_t)k;
  if (!par || !skip_root_heads) return par != 0;
  std::vector<char> root(img.tag.size(), 0);
  for (uint32_t r : img.roots)
    if (r >= IMG_FIRST) root[r - IMG_FIRST] = 1;
  for (size_t k = 0; k < img.tag.size(); ++k)
    if ((img.tag[k] & KIND_MASK) == K_CONS && !root[k] && (uint32_t)img.word[k] == par) return true;
  return false;
}
// Is there a wide list (a data list or (list ...) with >= WIDE_MIN elements after its head) below the top
// level that is not the operand of a quote?  Its evaluation may suspend (nested mode, NEST_EVAL).  Reader
// spines are contiguous (c.14): cell k continues a list iff cell k-1 is a cons whose cdr is k.
static bool image_has_wide_nested(const Image& img) {
  size_t N = img.tag.size();
  auto is_cons = [&](size_t k) { return (img.tag[k] & KIND_MASK) == K_CONS; };
  std::vector<uint32_t> cand;                         // starts (image-local) of runs of >= WIDE_MIN + 1 cells
  size_t start = 0, run = 0;
  for (size_t k = 0; k < N; ++k) {
    if (!is_cons(k)) { run = 0; continue; }
    if (run && (uint32_t)(img.word[k - 1] >> 32) == IMG_FIRST + k) {
      ++run;
    } else {
      start = k;
      run = 1;
    }
    if (run == WIDE_MIN + 1) cand.push_back(IMG_FIRST + (uint32_t)start);
  }
  if (cand.empty()) return false;                     // (the common case: one pass, nothing allocated)
  std::vector<char> skip(cand.size(), 0);             // candidates that are top-level forms or quoted
  auto mark = [&](uint32_t x) {
    auto it = std::lower_bound(cand.begin(), cand.end(), x);
    if (it != cand.end() && *it == x) skip[it - cand.begin()] = 1;
  };
  for (uint32_t r : img.roots) mark(r);
  for (size_t k = 0; k < N; ++k) {                    // (quote x): x is not evaluated
    if (!is_cons(k)) continue;
    uint32_t h = (uint32_t)img.word[k], c2 = (uint32_t)(img.word[k] >> 32);
    if (h < IMG_FIRST || (img.tag[h - IMG_FIRST] & KIND_MASK) != K_SYM || img.word[h - IMG_FIRST] != SP_QUOTE) continue;
    if (c2 < IMG_FIRST || !is_cons(c2 - IMG_FIRST)) continue;
    mark((uint32_t)img.word[c2 - IMG_FIRST]);
  }
  for (char s : skip)
    if (!s) return true;
  return false;
}
static bool image_mentions_setq(const Image& img) {
  for (size_t k = 0; k < img.tag.size(); ++k)
    if ((img.tag[k] & KIND_MASK) == K_SYM && img.word[k] == SP_SETQ) return true;
  return false;
}
// Closures are made only by lambda and defun (c.4): without either symbol there is no closure to apply,
// so argument splitting (which polls at closure calls) cannot help and the eval grid can shrink.
static bool image_mentions_closure(const Image& img) {
  for (size_t k = 0; k < img.tag.size(); ++k)
    if ((img.tag[k] & KIND_MASK) == K_SYM && (img.word[k] == SP_LAMBDA || img.word[k] == SP_DEFUN)) return true;
  return false;
}
static EvalArgs make_args(culi_ctx* c, uint32_t nforms, const uint32_t* perm, int define_mode) {
  EvalArgs A{};
  A.H = c->H;
  A.kst = c->kst;
  A.vst = c->vst;
  A.nslots = c->nslots;
  A.stride = c->nslots * (uint32_t)sizeof(uint4);
  A.kcap = c->kcap;
  A.vcap = c->vcap;
  A.roots = c->roots.p;
  A.perm = perm;
  A.nforms = nforms;
  A.next = c->next;
  A.rtag = c->rtag.p;
  A.rerr = c->rerr.p;
  A.rsteps = c->rsteps.p;
  A.rword = c->rword.p;
  A.max_depth = c->opts.max_depth;
  A.fuel = c->opts.fuel;
  A.define_mode = define_mode;
  A.flags = c->flags;
  A.voting = (c->opts.flags & CULI_F_NO_VOTING) ? 0 : 1;
  A.lanes = 32;
  A.fanout = (!define_mode && !(c->opts.flags & CULI_F_NO_FANOUT)) ? 1 : 0;
  A.desc = c->desc;
  A.npend = c->npend;
  A.maxdesc = c->maxdesc;
  A.fallback = c->fallback.p;
  A.nfallback = c->nfallback;
  A.wide = (!define_mode && c->batch_has_wide) ? c->wide.p : nullptr;
  A.nest = (!define_mode && c->batch_may_nest && c->kst2 && !(c->opts.flags & CULI_F_NO_NESTED)) ? 1 : 0;
  A.ndesc = c->ndesc;
  A.nnest = c->nnest;
  A.maxnest = c->maxnest;
  A.kst2 = c->kst2;
  A.vst2 = c->vst2;
  A.finished = c->nnest + 1;
  // argument splitting: where a closure may be applied (the poll sits at closure calls), binned or not
  (void)perm;
  // (a batch that is one top-level ||| form spends its time in the fan-out kernel: its eval launch needs one
  // block, not a grid of idle thieves — C3 eval phase 0.19 -> 0.165 ms)
  A.split = (!define_mode && c->batch_may_close && !(c->opts.flags & CULI_F_NO_SPLIT) &&
             !(c->batch_single_par && !(c->opts.flags & CULI_F_NO_FANOUT))) ? 1 : 0;
  // setq (R7): frames go to the heap when made, and a form runs in one thread only (no fan-out, nested
  // fan-out or argument splitting: those evaluate parts of a form elsewhere, on copies of its frames)
  A.mut = define_mode ? c->define_mut : c->batch_mut;
  A.pmark = (uint32_t)c->mark;
  if (A.mut && !define_mode) {
    A.fanout = 0;
    A.nest = 0;
    A.split = 0;
    A.wide = nullptr;
  }
  A.split_poll = c->split_poll;
  A.split_first = c->split_first;
  A.steal_gate = c->steal_gate;
  A.split_sleep = c->split_sleep;
  A.groups = c->groups;
  A.gqueue = c->gqueue;
  A.gqcap = c->gqcap;
  A.sctl = c->sctl;
  A.wait_ns = c->wait_ns;
  A.payload = c->payload.p;
  A.pcount = c->pcount;
  A.pcap = c->payload.n;
  // stage the persistent code segment and the global frame in shared memory (batch mode only)
  bool stage = !define_mode && !(c->opts.flags & CULI_F_NO_STAGING);
  A.code_lo = IMG_FIRST;
  A.code_n = (stage && CULI_STAGE_CODE) ? (uint32_t)std::min<uint64_t>(c->mark - IMG_FIRST, 1536) : 0;
  A.gst = stage ? (uint32_t)std::min<size_t>(c->syms->names.size(), 2048) : 0;
  return A;
}

// H2D of an image into the heap at c->mark (strings after the persistent strings) + relocation.
static int upload_image(culi_ctx* c, const Image& img, uint32_t str_base) {
  uint64_t n = img.tag.size();
  if (c->mark + n > c->H.cap) return CULI_E_HEAP_FULL;
  if (img.max_sym > c->H.gcap || c->syms->names.size() > c->H.gcap) return CULI_E_HEAP_FULL;
  if ((uint64_t)str_base + img.strings.size() > c->str_cap) return CULI_E_HEAP_FULL;
  uint32_t nr = (uint32_t)img.roots.size();
  CK(c->roots.ensure(std::max<uint32_t>(nr, 1)));
  size_t tw = (n + 7) / 8;                           // staging: word[] at [0, n), tag[] after it
  if (n) {
    CK(c->stage.ensure(n + tw));
    CK(cudaMemcpyAsync(c->stage.p, img.word.data(), n * 8, cudaMemcpyHostToDevice, c->stream));
    CK(cudaMemcpyAsync(c->stage.p + n, img.tag.data(), n, cudaMemcpyHostToDevice, c->stream));
  }
  if (!img.strings.empty())
    CK(cudaMemcpyAsync((char*)c->H.strs + str_base, img.strings.data(), img.strings.size(),
                       cudaMemcpyHostToDevice, c->stream));
  if (nr) CK(cudaMemcpyAsync(c->roots.p, img.roots.data(), nr * 4, cudaMemcpyHostToDevice, c->stream));
  CK(launch_relocate(c->stream, (const uint8_t*)(c->stage.p + n), c->stage.p, c->H.tag.p, c->mark, n, str_base,
                     c->roots.p, nr, c->sms));
  if (!img.wide_len.empty()) {                       // wide lists: their element count in O(1) (TAG_LEN)
    uint32_t np = (uint32_t)(img.wide_len.size() / 2);
    CK(c->lenpairs.ensure(2 * np));
    CK(cudaMemcpyAsync(c->lenpairs.p, img.wide_len.data(), 8ull * np, cudaMemcpyHostToDevice, c->stream));
    CK(launch_lenmark(c->stream, c->H.tag.p, c->mark, c->lenpairs.p, np));
  }
  return CULI_OK;
}

static int ensure_results(culi_ctx* c, uint32_t nforms) {
  size_t n = std::max<uint32_t>(nforms, 1);
  CK(c->rtag.ensure(n));
  CK(c->rerr.ensure(n));
  CK(c->rsteps.ensure(n));
  CK(c->rword.ensure(n));
  return CULI_OK;
}

static int run_collect(culi_ctx* c) {
  uint64_t live = 0, freed = 0;
  int rc = collect_persistent(c, &live, &freed);
  if (rc) return rc;
  c->gc.last_live = live;
  c->gc.last_freed = freed;
  c->gc.total_freed += freed;
  ++c->gc.collections;
  return CULI_OK;
}

// Evaluate the nf definition forms already in the heap at c->mark (nnodes image nodes), in order.
static int run_define(culi_ctx* c, uint32_t nf, uint64_t nnodes, uint32_t* failed_index, uint8_t* failed_err) {
  int rc = ensure_results(c, nf);
  if (rc) return rc;
  CK(launch_reset(c->stream, c->H.top, c->mark + nnodes, c->next, c->pcount, c->flags, c->npend,
                  c->nfallback, c->nnest, c->sctl));
  EvalArgs A = make_args(c, nf, nullptr, 1);
  if (nf) CK(launch_define(c->stream, A));
  int flags[8];
  unsigned long long top = 0;
  CK(cudaMemcpyAsync(flags, c->flags, sizeof flags, cudaMemcpyDeviceToHost, c->stream));
  CK(cudaMemcpyAsync(&top, c->H.top, 8, cudaMemcpyDeviceToHost, c->stream));
  CK(cudaStreamSynchronize(c->stream));
  c->mark = std::min<unsigned long long>(top, c->H.cap);
  c->heap_high = std::max<uint64_t>(c->heap_high, top);
  c->defined = true;
  // reclaim the persistent segment: keep what the global frame reaches (§8(f)3, culi_gc.cu)
  if (!(c->opts.flags & CULI_F_NO_GC)) {
    int g = run_collect(c);
    if (g) return g;
  }
  if (flags[0] && !flags[1]) return CULI_E_HEAP_FULL;
  if (flags[1]) {
    if (failed_index) *failed_index = (uint32_t)(flags[1] - 1);
    if (failed_err) *failed_err = (uint8_t)flags[2];
    if (flags[2] == E_OOM) return CULI_E_HEAP_FULL;
    return CULI_E_DEFINE;
  }
  return CULI_OK;
}

extern "C" int culi_define(culi_ctx* c, const culi_image* defs, uint32_t* failed_index,
                           uint8_t* failed_err) {
  if (!c || !defs) return CULI_E_ARG;
  if (c->have_batch || c->pending) return CULI_E_STATE;   // definitions go below an uploaded batch: release it first
  const Image& img = defs->img;
  uint32_t nf = (uint32_t)img.roots.size();
  uint32_t str_base = (uint32_t)c->strings.size();
  int rc = upload_image(c, img, str_base);
  if (rc) return rc;
  c->strings += img.strings;
  c->persist_has_par = c->persist_has_par || image_mentions_par(img) || image_has_wide_nested(img);
  c->persist_has_closure = c->persist_has_closure || image_mentions_closure(img);
  c->define_mut = c->persist_has_setq || image_mentions_setq(img);
  c->persist_has_setq = c->define_mut;
  return run_define(c, nf, img.tag.size(), failed_index, failed_err);
}

extern "C" int culi_define_text(culi_ctx* c, const char* text, size_t len, int text_on_device,
                                uint32_t* failed_index, uint8_t* failed_err, size_t* err_offset) {
  if (!c || (!text && len)) return CULI_E_ARG;
  if (c->have_batch || c->pending) return CULI_E_STATE;
  ReadOut ro;
  int rc = device_read(c, text, len, text_on_device != 0, &ro, err_offset);
  if (rc) return rc;
  c->strings += ro.strings;
  c->persist_has_par = c->persist_has_par || ro.par_root_head || ro.par_nested || ro.wide_nested;
  c->persist_has_closure = c->persist_has_closure || ro.closure;
  c->define_mut = c->persist_has_setq || ro.setq;
  c->persist_has_setq = c->define_mut;
  return run_define(c, ro.nforms, ro.nodes, failed_index, failed_err);
}

// Phase timing events; while the step is being captured into a graph they become external event-record
// nodes, so culi_last_timing also works after a replay.
static cudaError_t record_event(culi_ctx* c, int k) {
  cudaStreamCaptureStatus st = cudaStreamCaptureStatusNone;
  if (c->stream) cudaStreamIsCapturing(c->stream, &st);
  if (st == cudaStreamCaptureStatusActive) return cudaEventRecordWithFlags(c->ev[k], c->stream, cudaEventRecordExternal);
  return cudaEventRecord(c->ev[k], c->stream);
}

// Run dispatch + eval + export for the uploaded batch (device only, stream-ordered, no host sync).
static int run_batch_device(culi_ctx* c) {
  uint32_t nf = c->batch_forms;
  c->last_kernels = 0;
  CK(record_event(c, 0));
  CK(launch_reset(c->stream, c->H.top, c->mark + c->batch_nodes, c->next, c->pcount, c->flags, c->npend,
                  c->nfallback, c->nnest, c->sctl));
  ++c->last_kernels;
  uint32_t* perm = nullptr;
  if (!(c->opts.flags & CULI_F_NO_BINNING) && nf > 1 && (nf >= BIN_MIN_FORMS || c->batch_may_close)) {
    // closure-free batches (the voting kernel): biggest forms first (CULI_SIZE_FIRST=0 turns it off)
    uint32_t size_first = !c->batch_may_close && c->size_first;
    CK(launch_dispatch(c->stream, c->H, c->roots.p, nf, c->keys.p, c->keys_alt.p, c->perm.p,
                       c->perm_alt.p, c->dtemp.p, c->dtemp.n, &perm, c->sms, size_first));
    c->last_kernels += dispatch_launches(nf);
  }
  CK(record_event(c, 1));
  EvalArgs A = make_args(c, nf, perm, 0);
  A.fanout = A.fanout && c->batch_has_par;
  // small unbinned batches (<= 128 warps, fewer than the SMs) are latency-bound: the voting kernel's
  // regrouping costs more than the divergence it saves there (C1: 0.056 -> 0.049 ms eval)
  if (nf < BIN_MIN_FORMS) A.voting = 0;
  if (A.nest) { CK(launch_nest_clear(c->stream, c->ndesc, c->maxnest)); ++c->last_kernels; }
  uint32_t blocks = c->nslots / 128;
  uint32_t need = (nf + 127) / 128;
  // a batch that may suspend on nested ||| or split arguments keeps the whole grid: idle warps apply the
  // elements / evaluate split-off arguments
  if (need < blocks && !A.nest && !A.split) blocks = std::max<uint32_t>(need, 1);
  // a small batch on the plain kernel is latency-bound and its lanes diverge (different forms): thin warps
  // — `lanes` forms per warp, about one warp per scheduler of the GPU — serialise fewer paths per warp
  A.lanes = 32;
  if (!A.nest && !A.split && nf < BIN_MIN_FORMS) {
    uint32_t want = (nf + 4 * c->sms - 1) / (4 * c->sms), lanes = 1;
    while (lanes < want && lanes < 32) lanes *= 2;
    if (c->thin_lanes) lanes = c->thin_lanes;
    A.lanes = lanes;
    blocks = std::min<uint32_t>(c->nslots / 128, std::max<uint32_t>((nf + 4 * lanes - 1) / (4 * lanes), 1));
  }
  // kernels bounded at CULI_BLOCKS_PER_SM resident blocks (voting, plain, fan-out) get one wave at most; they
  // take their work from counters, so a smaller grid only means fewer, fuller threads
  const uint32_t one_wave = (uint32_t)c->sms * CULI_BLOCKS_PER_SM;
  if (!A.nest && !A.split) blocks = std::min(blocks, one_wave);
  if (nf) { CK(launch_eval(c->stream, A, blocks)); ++c->last_kernels; }
  if (nf && A.fanout && c->batch_has_par) {            // ||| fan-out (a6) + finalize (a8)
    CK(launch_fanout(c->stream, A, std::min(c->nslots / 128, one_wave)));
    c->last_kernels += 2;
  }
  CK(record_event(c, 2));
  ExportArgs X{};
  X.tag = c->H.tag;
  X.word = c->H.word;
  X.rtag = c->rtag.p;
  X.rword = c->rword.p;
  X.nforms = nf;
  X.vst = c->vst;
  X.nslots = c->nslots;
  X.vcap = c->vcap;
  X.payload = c->payload.p;
  X.pcount = c->pcount;
  X.pcap = c->payload.n;
  X.flags = c->flags;
  X.list = nullptr;
  X.nlist = 0;
  if (nf) { CK(launch_export(c->stream, X, blocks)); ++c->last_kernels; }
  if (nf && A.fanout && c->batch_has_par) {
    CK(launch_flat_export(c->stream, A, c->sms * 8));
    c->last_kernels += 2;
  }
  CK(record_event(c, 3));
  return CULI_OK;
}

// Buffers and launch decisions for a batch whose image is already in the heap at c->mark (uploaded from a
// host image or written by the device reader).  par_any / par_nonroot: the ||| symbol is the car of some
// cell / of some cell other than a top-level form's first cell; par_head: some form is (||| ...).
static int finish_prepare(culi_ctx* c, uint32_t nf, uint64_t nnodes, std::string strings, bool par_any,
                          bool par_nonroot, bool par_head, bool has_wide, bool setq, bool closure) {
  c->batch_mut = c->persist_has_setq || setq;
  c->batch_may_close = c->persist_has_closure || closure;
  drop_graph(c);
  int rc = ensure_results(c, nf);
  if (rc) return rc;
  size_t n = std::max<uint32_t>(nf, 1);
  CK(c->keys.ensure(2 * n));                         // 64-bit dispatch keys
  CK(c->keys_alt.ensure(2 * n));
  CK(c->perm.ensure(n));
  CK(c->perm_alt.ensure(n));
  CK(c->dtemp.ensure(dispatch_temp_bytes(nf)));
  // tokens: ~4 per form; a ||| result list can be as long as the persistent segment (2 tokens per cell)
  CK(c->payload.ensure(std::max<size_t>(4 * (size_t)nf + 2 * (size_t)(c->mark + nnodes), 1 << 16)));
  c->have_batch = true;
  c->batch_nodes = nnodes;
  c->batch_forms = nf;
  c->batch_strings = std::move(strings);
  CK(c->fallback.ensure((size_t)c->maxdesc + nf + 1));
  // may ||| occur below the top level (nested fan-out, §8(f)1)?  any ||| symbol in the batch or in a definition
  c->batch_may_nest = c->persist_has_par || ((c->opts.flags & CULI_F_NO_FANOUT) ? par_any : par_nonroot);
  if (c->batch_may_nest && !c->kst2 && !(c->opts.flags & CULI_F_NO_NESTED)) {
    CK(cudaMalloc(&c->kst2, (size_t)c->nslots * c->kcap * sizeof(uint4)));
    CK(cudaMalloc(&c->vst2, (size_t)c->nslots * c->vcap * sizeof(uint4)));
  }
  c->batch_has_par = par_head;
  c->batch_single_par = nf == 1 && par_head;
  c->batch_has_wide = has_wide;
  if (has_wide) c->batch_has_par = true;             // the fan-out kernels handle both
  return CULI_OK;
}

static int prepare_batch(culi_ctx* c, const Image& img) {
  uint32_t nf = (uint32_t)img.roots.size();
  uint32_t str_base = (uint32_t)c->strings.size();
  int rc = upload_image(c, img, str_base);
  if (rc) return rc;
  // does any form start with the ||| symbol (a6), or have >= WIDE_MIN arguments (wide forms, K12)?
  bool par_head = false, has_wide = false;
  std::vector<uint32_t> wide;
  for (uint32_t f = 0; f < nf; ++f) {
    uint32_t r = img.roots[f];
    if (r < IMG_FIRST || (img.tag[r - IMG_FIRST] & KIND_MASK) != K_CONS) continue;
    uint64_t rw = img.word[r - IMG_FIRST];
    uint32_t h = (uint32_t)rw;
    if (h >= IMG_FIRST && (img.tag[h - IMG_FIRST] & KIND_MASK) == K_SYM &&
        img.word[h - IMG_FIRST] == N_SPECIALS + BI_PAR)
      par_head = true;
    uint32_t nargs = 0;
    for (uint32_t q = (uint32_t)(rw >> 32); q >= IMG_FIRST; q = (uint32_t)(img.word[q - IMG_FIRST] >> 32)) ++nargs;
    if (nargs >= WIDE_MIN) {
      if (wide.empty()) wide.assign(nf, 0);
      wide[f] = nargs;
      has_wide = true;
    }
  }
  if (has_wide) {
    CK(c->wide.ensure(nf));
    CK(cudaMemcpyAsync(c->wide.p, wide.data(), nf * 4, cudaMemcpyHostToDevice, c->stream));
  }
  bool wide_nested = image_has_wide_nested(img);      // (counts as a nested ||| for the launch mode)
  return finish_prepare(c, nf, img.tag.size(), img.strings, image_mentions_par(img, false) || wide_nested,
                        image_mentions_par(img, true) || wide_nested, par_head, has_wide, image_mentions_setq(img),
                        image_mentions_closure(img));
}

// Device reader (§8(f)2) -> the same prepared batch.
// Host text up to this size is read by the host reader in culi_eval_text / culi_upload_text:
// a read of a few KB costs ~0.2 ms of device-reader launches and sync points, ~0.03-0.17 ms on the host.
constexpr size_t HOST_READ_MAX = 16384;
static int prepare_text(culi_ctx* c, const char* text, size_t len, bool on_device, size_t* err_offset) {
  if (!on_device && len <= HOST_READ_MAX && !(c->opts.flags & CULI_F_DEVICE_READ) && !c->force_device_read) {
    Image img;                                       // small host text: the host reader is faster here
    int rc = read_image(*c->syms, text, len, img, err_offset);
    if (rc) return rc;
    return prepare_batch(c, img);
  }
  ReadOut ro;
  int rc = device_read(c, text, len, on_device, &ro, err_offset);
  if (rc) return rc;
  return finish_prepare(c, ro.nforms, ro.nodes, std::move(ro.strings),
                        ro.par_root_head || ro.par_nested || ro.wide_nested, ro.par_nested || ro.wide_nested,
                        ro.par_root_head, ro.wide, ro.setq, ro.closure);
}

// ||| forms the fan-out could not decide (an element error, fuel overflow, a short or non-contiguous
// list) are re-evaluated exactly, one thread per form, without fan-out; then exported.
static int rerun_fallback(culi_ctx* c, uint32_t nfb) {
  CK(cudaMemsetAsync(c->next, 0, sizeof(uint32_t), c->stream));
  EvalArgs A = make_args(c, nfb, c->fallback.p, 0);
  A.fanout = 0;
  A.nest = 0;
  A.split = 0;
  CK(launch_eval(c->stream, A, std::max<uint32_t>(1, std::min<uint32_t>(std::min<uint32_t>(c->nslots / 128,
                                                                                 (uint32_t)c->sms * CULI_BLOCKS_PER_SM),
                                                                        (nfb + 127) / 128))));
  ExportArgs X{};
  X.tag = c->H.tag;
  X.word = c->H.word;
  X.rtag = c->rtag.p;
  X.rword = c->rword.p;
  X.nforms = c->batch_forms;
  X.vst = c->vst;
  X.nslots = c->nslots;
  X.vcap = c->vcap;
  X.payload = c->payload.p;
  X.pcount = c->pcount;
  X.pcap = c->payload.n;
  X.flags = c->flags;
  X.list = c->fallback.p;
  X.nlist = nfb;
  CK(launch_export(c->stream, X, std::max<uint32_t>(1, (nfb + 127) / 128)));
  CK(cudaMemsetAsync(c->nfallback, 0, sizeof(uint32_t), c->stream));
  return CULI_OK;
}

// Finish the device-resident results of the current batch: sequential fallbacks of undecided ||| forms,
// eval + export again into a grown payload buffer.  Synchronises.  *pc = payload tokens.
static int complete_device(culi_ctx* c, unsigned long long* pc_out) {
  for (int attempt = 0; attempt < 4; ++attempt) {
    int flags[8];
    unsigned long long pc = 0, top = 0;
    uint32_t nfb = 0, npend = 0, nnest = 0;
    SplitCtl sc{};
    CK(cudaMemcpyAsync(&npend, c->npend, 4, cudaMemcpyDeviceToHost, c->stream));
    if (attempt == 0) CK(cudaMemcpyAsync(&sc, c->sctl, sizeof sc, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaMemcpyAsync(&nnest, c->nnest, 4, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaMemcpyAsync(flags, c->flags, sizeof flags, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaMemcpyAsync(&pc, c->pcount, 8, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaMemcpyAsync(&top, c->H.top, 8, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaMemcpyAsync(&nfb, c->nfallback, 4, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaStreamSynchronize(c->stream));
    c->heap_high = std::max<uint64_t>(c->heap_high, std::min<unsigned long long>(top, c->H.cap));
    if (flags[0] || flags[4]) return CULI_E_HEAP_FULL;
    if (attempt == 0) {
      c->last_regrows = 0;
      c->last_fanout = (c->batch_has_par && !(c->opts.flags & CULI_F_NO_FANOUT)) ? std::min(npend, c->maxdesc) : 0;
      c->last_fallback = 0;
      c->last_nested = c->batch_may_nest ? std::min(nnest, c->maxnest) : 0;
      c->last_splits = sc.published;
      c->last_timeouts = sc.timeouts;
      c->last_claimed = sc.claimed;
      if (getenv("CULI_SPLIT_STATS"))
        fprintf(stderr, "[culi split] groups published %u claimed %u; idle rounds %u (lanes missing %u)\n",
                sc.published, sc.claimed, sc.stat[0], sc.stat[1]);
      std::memcpy(c->last_diag, sc.diag, sizeof sc.diag);
#if CULI_WATCHDOG
      if (sc.wd[0]) fprintf(stderr, "[culi watchdog] %u lanes fired; first: form %u steps(lo) %u sp %u depth %u root %u thief %u finished %u\n",
                            sc.wd[0], sc.wd[1], sc.wd[2], sc.wd[3], sc.wd[4], sc.wd[5], sc.wd[6], sc.wd[7]);
#endif
    }
    if (nfb && !flags[3]) {
      c->last_fallback += nfb;
      int rc = rerun_fallback(c, nfb);
      if (rc) return rc;
      continue;
    }
    if (flags[3]) {                                  // payload buffer too small: grow, re-export
      ++c->last_regrows;
      drop_graph(c);                                 // a captured step still points at the old buffer
      CK(c->payload.ensure((size_t)pc + 1024));
      int zero[8] = {0};
      CK(cudaMemcpyAsync(c->flags, zero, sizeof zero, cudaMemcpyHostToDevice, c->stream));
      CK(cudaMemsetAsync(c->pcount, 0, 8, c->stream));
      // results' words were partially rewritten: export reads rword as node index only for records
      // that were not yet exported, so re-run eval + export from scratch
      int rc = run_batch_device(c);
      if (rc) return rc;
      continue;
    }
    *pc_out = pc;
    return CULI_OK;
  }
  return CULI_E_HEAP_FULL;
}

// complete_device + D2H of records and payload into a new results object
static int fetch(culi_ctx* c, culi_results** out) {
  uint32_t nf = c->batch_forms;
  unsigned long long pc = 0;
  int rc = complete_device(c, &pc);
  if (rc) return rc;
  {
    culi_results* r = new (std::nothrow) culi_results;
    if (!r) return CULI_E_ARG;
    r->r.resize(nf);
    if (nf) {                                        // straight into the result arrays
      CK(cudaMemcpyAsync(r->r.tag.data(), c->rtag.p, nf, cudaMemcpyDeviceToHost, c->stream));
      CK(cudaMemcpyAsync(r->r.err.data(), c->rerr.p, nf, cudaMemcpyDeviceToHost, c->stream));
      CK(cudaMemcpyAsync(r->r.steps.data(), c->rsteps.p, nf * 8, cudaMemcpyDeviceToHost, c->stream));
      CK(cudaMemcpyAsync(r->r.word.data(), c->rword.p, nf * 8, cudaMemcpyDeviceToHost, c->stream));
    }
    static_assert(sizeof(Token) == sizeof(uint4), "token layout = device uint4 {word.lo, word.hi, tag, 0}");
    r->r.payload.resize(pc);
    if (pc) CK(cudaMemcpyAsync(r->r.payload.data(), c->payload.p, pc * sizeof(uint4), cudaMemcpyDeviceToHost, c->stream));
    CK(cudaStreamSynchronize(c->stream));
    r->r.syms = c->syms;
    r->r.strings = c->strings + c->batch_strings;
    *out = r;
    return CULI_OK;
  }
}

extern "C" {

int culi_eval_batch_async(culi_ctx* c, const culi_image* forms, culi_results** out) {
  if (!c || !forms || !out) return CULI_E_ARG;
  *out = nullptr;
  if (c->pending || c->have_batch) return CULI_E_STATE;
  culi_results* r = new (std::nothrow) culi_results;
  if (!r) return CULI_E_ARG;
  int rc = prepare_batch(c, forms->img);
  if (!rc) rc = run_batch_device(c);
  if (rc) {
    c->have_batch = false;
    delete r;
    return rc;
  }
  r->ready = false;
  r->owner = c;
  c->pending = r;
  *out = r;
  return CULI_OK;
}

int culi_sync(culi_ctx* c) {
  if (!c) return CULI_E_ARG;
  if (!c->pending) return cudaStreamSynchronize(c->stream) == cudaSuccess ? CULI_OK : CULI_E_CUDA;
  culi_results* p = c->pending;
  c->pending = nullptr;
  culi_results* tmp = nullptr;
  int rc = fetch(c, &tmp);
  c->have_batch = false;
  p->owner = nullptr;
  if (rc) return rc;                                 // p stays not ready
  p->r = std::move(tmp->r);
  p->ready = true;
  delete tmp;
  return CULI_OK;
}

int culi_complete(culi_ctx* c, uint32_t handle) {
  if (!c || handle != 1 || !c->have_batch) return CULI_E_STATE;
  unsigned long long pc = 0;
  return complete_device(c, &pc);
}

int culi_eval_batch(culi_ctx* c, const culi_image* forms, culi_results** out) {
  if (!c || !forms || !out) return CULI_E_ARG;
  *out = nullptr;
  if (c->pending) return CULI_E_STATE;
  int rc = prepare_batch(c, forms->img);
  if (rc) return rc;
  rc = run_batch_device(c);
  if (rc) return rc;
  rc = fetch(c, out);
  c->have_batch = false;
  return rc;
}

int culi_eval_text(culi_ctx* c, const char* text, size_t len, int text_on_device, culi_results** out,
                   size_t* err_offset) {
  if (!c || !out || (!text && len)) return CULI_E_ARG;
  if (c->pending) return CULI_E_STATE;
  *out = nullptr;
  int rc = prepare_text(c, text, len, text_on_device != 0, err_offset);
  if (rc) return rc;
  rc = run_batch_device(c);
  if (rc) return rc;
  rc = fetch(c, out);
  c->have_batch = false;
  return rc;
}

int culi_upload_text(culi_ctx* c, const char* text, size_t len, int text_on_device, uint32_t* handle,
                     uint32_t* nforms, size_t* err_offset) {
  if (!c || (!text && len)) return CULI_E_ARG;
  if (c->pending) return CULI_E_STATE;
  int rc = prepare_text(c, text, len, text_on_device != 0, err_offset);
  if (rc) return rc;
  if (handle) *handle = 1;
  if (nforms) *nforms = c->batch_forms;
  return CULI_OK;
}

int culi_collect(culi_ctx* c, uint64_t* live_nodes, uint64_t* freed_nodes) {
  if (!c) return CULI_E_ARG;
  if (c->have_batch) return CULI_E_STATE;
  int rc = run_collect(c);
  if (rc) return rc;
  if (live_nodes) *live_nodes = c->gc.last_live;
  if (freed_nodes) *freed_nodes = c->gc.last_freed;
  return CULI_OK;
}

int culi_heap_usage(const culi_ctx* c, uint64_t* persistent_nodes, uint64_t* capacity, uint64_t* freed_total) {
  if (!c) return CULI_E_ARG;
  if (persistent_nodes) *persistent_nodes = c->mark;
  if (capacity) *capacity = c->H.cap;
  if (freed_total) *freed_total = c->gc.total_freed;
  return CULI_OK;
}

int culi_last_read(const culi_ctx* c, float* ms, uint64_t* items, uint64_t* nodes) {
  if (!c) return CULI_E_ARG;
  if (ms) *ms = c->rd.last_ms;
  if (items) *items = c->rd.last_items;
  if (nodes) *nodes = c->rd.last_nodes;
  return CULI_OK;
}

int culi_upload(culi_ctx* c, const culi_image* forms, uint32_t* handle) {
  if (!c || !forms) return CULI_E_ARG;
  if (c->pending) return CULI_E_STATE;
  int rc = prepare_batch(c, forms->img);
  if (rc) return rc;
  CK(cudaStreamSynchronize(c->stream));
  if (handle) *handle = 1;
  return CULI_OK;
}

// Repeated evaluation of one uploaded batch replays a CUDA graph of the whole device step (reset, dispatch,
// eval, fan-out, export: ~10 launches), captured on the first call; small batches are launch-bound.
// The legacy default stream cannot be captured: there the launches are issued directly.
int culi_eval_uploaded(culi_ctx* c, uint32_t handle) {
  if (!c || handle != 1 || !c->have_batch) return CULI_E_STATE;
  if (!c->stream || (c->opts.flags & CULI_F_NO_GRAPH)) return run_batch_device(c);
  if (!c->graph_exec) {
    CK(cudaStreamBeginCapture(c->stream, cudaStreamCaptureModeThreadLocal));
    int rc = run_batch_device(c);
    cudaGraph_t g = nullptr;
    cudaError_t e = cudaStreamEndCapture(c->stream, &g);
    if (rc || e != cudaSuccess || !g) {
      if (g) cudaGraphDestroy(g);
      return rc ? rc : CULI_E_CUDA;
    }
    // the exact number of kernels one step launches: the kernel nodes of the captured graph (the library
    // sort picks its kernels by size, so counting launch calls would only estimate it)
    size_t nn = 0;
    uint32_t kn = 0;
    if (cudaGraphGetNodes(g, nullptr, &nn) == cudaSuccess && nn) {
      std::vector<cudaGraphNode_t> nodes(nn);
      if (cudaGraphGetNodes(g, nodes.data(), &nn) == cudaSuccess)
        for (size_t q = 0; q < nn; ++q) {
          cudaGraphNodeType ty;
          if (cudaGraphNodeGetType(nodes[q], &ty) == cudaSuccess && ty == cudaGraphNodeTypeKernel) ++kn;
        }
    }
    e = cudaGraphInstantiate(&c->graph_exec, g, 0);
    cudaGraphDestroy(g);
    if (e != cudaSuccess) {
      c->graph_exec = nullptr;
      return CULI_E_CUDA;
    }
    c->graph_kernels = kn ? kn : c->last_kernels;
  }
  CK(cudaGraphLaunch(c->graph_exec, c->stream));
  c->last_kernels = c->graph_kernels;
  return CULI_OK;
}

int culi_fetch_results(culi_ctx* c, uint32_t handle, culi_results** out) {
  if (!c || !out || handle != 1 || !c->have_batch) return CULI_E_STATE;
  *out = nullptr;
  return fetch(c, out);
}

int culi_release(culi_ctx* c, uint32_t handle) {
  if (!c || handle != 1) return CULI_E_STATE;
  drop_graph(c);
  c->have_batch = false;
  return CULI_OK;
}

int culi_records_device(culi_ctx* c, void* dev_buf, size_t cap, size_t* bytes) {
  if (!c) return CULI_E_ARG;
  size_t n = c->batch_forms;
  size_t o_steps = (2 * n + 7) & ~(size_t)7;
  size_t total = o_steps + 16 * n;
  if (bytes) *bytes = total;
  if (!dev_buf) return CULI_OK;
  if (cap < total || !c->have_batch) return CULI_E_ARG;
  char* d = (char*)dev_buf;
  if (n) {
    CK(cudaMemcpyAsync(d, c->rtag.p, n, cudaMemcpyDeviceToDevice, c->stream));
    CK(cudaMemcpyAsync(d + n, c->rerr.p, n, cudaMemcpyDeviceToDevice, c->stream));
    CK(cudaMemcpyAsync(d + o_steps, c->rsteps.p, 8 * n, cudaMemcpyDeviceToDevice, c->stream));
    CK(cudaMemcpyAsync(d + o_steps + 8 * n, c->rword.p, 8 * n, cudaMemcpyDeviceToDevice, c->stream));
  }
  return CULI_OK;
}

uint32_t culi_results_count(const culi_results* r) { return r && r->ready ? (uint32_t)r->r.size() : 0; }

int culi_result_info(const culi_results* r, uint32_t i, uint8_t* tag, uint8_t* err, uint64_t* steps) {
  if (r && !r->ready) return CULI_E_STATE;
  if (!r || i >= r->r.size()) return CULI_E_ARG;
  const Record x = r->r.at(i);
  if (tag) *tag = x.tag;
  if (err) *err = x.err;
  if (steps) *steps = x.steps;
  return CULI_OK;
}

int culi_result_int(const culi_results* r, uint32_t i, int64_t* v) {
  if (r && !r->ready) return CULI_E_STATE;
  if (!r || i >= r->r.size() || !v) return CULI_E_ARG;
  const Record x = r->r.at(i);
  if (x.err || x.tag != K_INT) return CULI_E_ARG;
  *v = (int64_t)x.word;
  return CULI_OK;
}

int culi_result_float(const culi_results* r, uint32_t i, double* v) {
  if (r && !r->ready) return CULI_E_STATE;
  if (!r || i >= r->r.size() || !v) return CULI_E_ARG;
  const Record x = r->r.at(i);
  if (x.err || x.tag != K_FLOAT) return CULI_E_ARG;
  std::memcpy(v, &x.word, 8);
  return CULI_OK;
}

int culi_print(const culi_results* r, uint32_t i, char* buf, size_t cap, size_t* needed) {
  if (r && !r->ready) return CULI_E_STATE;
  if (!r || i >= r->r.size()) return CULI_E_ARG;
  std::string s;
  r->r.print(i, s);
  if (needed) *needed = s.size();
  if (!buf || cap <= s.size()) {
    if (buf && cap) {
      std::memcpy(buf, s.data(), cap - 1);
      buf[cap - 1] = 0;
    }
    return CULI_E_ARG;
  }
  std::memcpy(buf, s.data(), s.size());
  buf[s.size()] = 0;
  return CULI_OK;
}

int culi_results_totals(const culi_results* r, uint64_t* total_steps, uint32_t* n_errors) {
  if (!r) return CULI_E_ARG;
  if (!r->ready) return CULI_E_STATE;
  uint64_t t = 0;
  uint32_t ne = 0;
  for (size_t q = 0; q < r->r.size(); ++q) {
    t += r->r.steps[q];
    ne += r->r.err[q] != 0;
  }
  if (total_steps) *total_steps = t;
  if (n_errors) *n_errors = ne;
  return CULI_OK;
}

void culi_results_free(culi_results* r) {
  if (r && !r->ready && r->owner) culi_sync(r->owner);   // finish the batch before its results go away
  delete r;
}

int culi_results_wire_bytes(const culi_results* r, uint64_t* d2h_bytes) {
  if (!r || !d2h_bytes) return CULI_E_ARG;
  if (!r->ready) return CULI_E_STATE;
  *d2h_bytes = r->r.size() * 18 + r->r.payload.size() * sizeof(Token);
  return CULI_OK;
}

int culi_last_stats(const culi_ctx* c, uint32_t* fanout_forms, uint32_t* fallback_forms,
                    uint32_t* nested_forms) {
  if (!c) return CULI_E_ARG;
  if (nested_forms) *nested_forms = c->last_nested;
  if (fanout_forms) *fanout_forms = c->last_fanout;
  if (fallback_forms) *fallback_forms = c->last_fallback;
  return CULI_OK;
}

int culi_last_splits(const culi_ctx* c, uint32_t* groups) {
  if (!c || !groups) return CULI_E_ARG;
  *groups = c->last_splits;
  return CULI_OK;
}

int culi_last_split_claims(const culi_ctx* c, uint32_t* claimed) {
  if (!c || !claimed) return CULI_E_ARG;
  *claimed = c->last_claimed;
  return CULI_OK;
}

int culi_last_reruns(const culi_ctx* c, uint32_t* fallback_forms, uint32_t* payload_regrows) {
  if (!c) return CULI_E_ARG;
  if (fallback_forms) *fallback_forms = c->last_fallback;
  if (payload_regrows) *payload_regrows = c->last_regrows;
  return CULI_OK;
}

int culi_last_waits(const culi_ctx* c, uint32_t* timeouts, uint32_t* diag9) {
  if (!c) return CULI_E_ARG;
  if (timeouts) *timeouts = c->last_timeouts;
  if (diag9) std::memcpy(diag9, c->last_diag, sizeof c->last_diag);
  return CULI_OK;
}

int culi_last_timing(const culi_ctx* c, float* ms3, uint32_t* kernels, uint64_t* heap_high) {
  if (!c) return CULI_E_ARG;
  if (ms3) {
    CK(cudaEventSynchronize(c->ev[3]));
    for (int k = 0; k < 3; ++k) CK(cudaEventElapsedTime(&ms3[k], c->ev[k], c->ev[k + 1]));
  }
  if (kernels) *kernels = c->last_kernels;
  if (heap_high) *heap_high = c->heap_high;
  return CULI_OK;
}

}  // extern "C"
