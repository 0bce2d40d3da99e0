// culi_dist.cu — distributed hooks of libculi.so.
//
// Env broadcast: rank 0 runs culi_define, packs the global environment into a device buffer
// (culi_env_export), the caller broadcasts it with NCCL (torch.distributed.broadcast over NVLink), and the
// other ranks unpack it (culi_env_import).  Heap indices are position-independent across ranks because
// every rank's persistent segment starts at node IMG_FIRST, so the segment is copied verbatim.
// Result gather: each rank serializes its results (records + payload + symbol names + string bytes); the
// caller all-gathers the blobs; culi_results_merge re-interns symbols by name and reorders by form index.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstring>
#include <memory>
#include <new>
#include <string>
#include <vector>

#include "../../include/culi.h"
#include "culi_ctx.h"

using namespace culi;

namespace {
constexpr uint64_t ENV_MAGIC = 0x31564e45494c5543ull;   // "CULIENV1"
constexpr uint64_t RES_MAGIC = 0x31534552494c5543ull;   // "CULIRES1"

struct EnvHeader {
  uint64_t magic;
  uint64_t mark;          // heap nodes [0, mark) of the persistent segment
  uint64_t nsyms;         // global table entries
  uint64_t nstr;          // string bytes
  uint64_t names_bytes;   // NUL-separated symbol names, id order
  uint64_t flags;         // bit 0: some definition mentions ||| (nested fan-out may be needed); bit 1: setq
  uint64_t pad[2];
};

inline uint64_t align8(uint64_t x) { return (x + 7) & ~7ull; }

struct EnvLayout {
  uint64_t o_node, o_gtag, o_gword, o_str, o_names, total;
  EnvLayout(const EnvHeader& h) {
    o_node = (sizeof(EnvHeader) + 15) & ~15ull;     // the persistent segment's 16-byte nodes, verbatim
    o_gtag = o_node + sizeof(Node) * h.mark;
    o_gword = align8(o_gtag + h.nsyms);
    o_str = o_gword + 8 * h.nsyms;
    o_names = o_str + h.nstr;
    total = align8(o_names + h.names_bytes);
  }
};

std::string names_blob(const SymTable& st) {
  std::string b;
  for (const auto& n : st.names) { b += n; b += '\0'; }
  return b;
}

#define CK(x)                                   \
  do {                                          \
    cudaError_t _e = (x);                       \
    if (_e != cudaSuccess) return CULI_E_CUDA;  \
  } while (0)

struct RecWire {
  uint64_t steps;
  uint64_t word;
  uint8_t tag;
  uint8_t err;
  uint8_t pad[6];
};
struct ResHeader {
  uint64_t magic, nforms, npayload, names_bytes, nstr, pad[3];
};
}  // namespace

extern "C" {

int culi_env_export(culi_ctx* c, void* dev_buf, size_t cap, size_t* bytes) {
  if (!c) return CULI_E_ARG;
  std::string names = names_blob(*c->syms);
  EnvHeader h{};
  h.magic = ENV_MAGIC;
  h.mark = c->mark;
  h.nsyms = c->syms->names.size();
  h.nstr = c->strings.size();
  h.names_bytes = names.size();
  h.flags = (c->persist_has_par ? 1 : 0) | (c->persist_has_setq ? 2 : 0) | (c->persist_has_closure ? 4 : 0);
  EnvLayout L(h);
  if (bytes) *bytes = L.total;
  if (!dev_buf || cap < L.total) return dev_buf ? CULI_E_ARG : CULI_OK;
  char* d = (char*)dev_buf;
  CK(cudaMemcpyAsync(d, &h, sizeof h, cudaMemcpyHostToDevice, c->stream));
  CK(cudaMemcpyAsync(d + L.o_node, c->H.tag.p, sizeof(Node) * h.mark, cudaMemcpyDeviceToDevice, c->stream));
  CK(cudaMemcpyAsync(d + L.o_gtag, c->H.gtag, h.nsyms, cudaMemcpyDeviceToDevice, c->stream));
  CK(cudaMemcpyAsync(d + L.o_gword, c->H.gword, 8 * h.nsyms, cudaMemcpyDeviceToDevice, c->stream));
  if (h.nstr) CK(cudaMemcpyAsync(d + L.o_str, c->H.strs, h.nstr, cudaMemcpyDeviceToDevice, c->stream));
  if (h.names_bytes)
    CK(cudaMemcpyAsync(d + L.o_names, names.data(), h.names_bytes, cudaMemcpyHostToDevice, c->stream));
  CK(cudaStreamSynchronize(c->stream));
  return CULI_OK;
}

int culi_env_import(culi_ctx* c, const void* dev_buf, size_t nbytes) {
  if (!c || !dev_buf || nbytes < sizeof(EnvHeader)) return CULI_E_ARG;
  if (c->defined || c->syms->names.size() != N_RESERVED) return CULI_E_STATE;
  const char* d = (const char*)dev_buf;
  EnvHeader h{};
  CK(cudaMemcpyAsync(&h, d, sizeof h, cudaMemcpyDeviceToHost, c->stream));
  CK(cudaStreamSynchronize(c->stream));
  if (h.magic != ENV_MAGIC) return CULI_E_ARG;
  EnvLayout L(h);
  if (L.total > nbytes) return CULI_E_ARG;
  if (h.mark > c->H.cap || h.nsyms > c->H.gcap || h.nstr > c->str_cap) return CULI_E_HEAP_FULL;
  std::string names(h.names_bytes, '\0');
  if (h.names_bytes)
    CK(cudaMemcpyAsync(&names[0], d + L.o_names, h.names_bytes, cudaMemcpyDeviceToHost, c->stream));
  CK(cudaMemcpyAsync(c->H.tag.p, d + L.o_node, sizeof(Node) * h.mark, cudaMemcpyDeviceToDevice, c->stream));
  CK(cudaMemcpyAsync(c->H.gtag, d + L.o_gtag, h.nsyms, cudaMemcpyDeviceToDevice, c->stream));
  CK(cudaMemcpyAsync(c->H.gword, d + L.o_gword, 8 * h.nsyms, cudaMemcpyDeviceToDevice, c->stream));
  if (h.nstr) CK(cudaMemcpyAsync((char*)c->H.strs, d + L.o_str, h.nstr, cudaMemcpyDeviceToDevice, c->stream));
  std::string strs(h.nstr, '\0');
  if (h.nstr) CK(cudaMemcpyAsync(&strs[0], d + L.o_str, h.nstr, cudaMemcpyDeviceToHost, c->stream));
  CK(cudaStreamSynchronize(c->stream));
  auto st = std::make_shared<SymTable>();
  size_t p = 0;
  uint32_t id = 0;
  while (p < names.size()) {
    size_t e = names.find('\0', p);
    if (e == std::string::npos) return CULI_E_ARG;
    if (st->intern(names.data() + p, e - p) != id) return CULI_E_ARG;   // reserved prefix must agree
    ++id;
    p = e + 1;
  }
  if (id != h.nsyms) return CULI_E_ARG;
  c->syms = st;
  c->strings = strs;
  c->mark = h.mark;
  c->persist_has_par = (h.flags & 1) != 0;
  c->persist_has_setq = (h.flags & 2) != 0;
  c->persist_has_closure = (h.flags & 4) != 0;
  c->defined = true;
  return CULI_OK;
}

int culi_results_serialize(const culi_results* r, void* buf, size_t cap, size_t* bytes) {
  if (!r) return CULI_E_ARG;
  if (!r->ready) return CULI_E_STATE;
  const Results& R = r->r;
  std::string names = names_blob(*R.syms);
  ResHeader h{};
  h.magic = RES_MAGIC;
  h.nforms = R.size();
  h.npayload = R.payload.size();
  h.names_bytes = names.size();
  h.nstr = R.strings.size();
  size_t total = sizeof h + h.nforms * sizeof(RecWire) + h.npayload * sizeof(Token) + h.names_bytes +
                 h.nstr;
  if (bytes) *bytes = total;
  if (!buf) return CULI_OK;
  if (cap < total) return CULI_E_ARG;
  char* p = (char*)buf;
  std::memcpy(p, &h, sizeof h);
  p += sizeof h;
  for (size_t q = 0; q < R.size(); ++q) {
    const Record x = R.at(q);
    RecWire w{};
    w.steps = x.steps;
    w.word = x.word;
    w.tag = x.tag;
    w.err = x.err;
    std::memcpy(p, &w, sizeof w);
    p += sizeof w;
  }
  if (h.npayload) std::memcpy(p, R.payload.data(), h.npayload * sizeof(Token));
  p += h.npayload * sizeof(Token);
  std::memcpy(p, names.data(), names.size());
  p += names.size();
  std::memcpy(p, R.strings.data(), R.strings.size());
  return CULI_OK;
}

int culi_results_merge(const void* const* blobs, const size_t* sizes, int nranks,
                       const uint32_t* const* form_index, culi_results** merged) {
  if (!blobs || !sizes || !form_index || !merged || nranks <= 0) return CULI_E_ARG;
  *merged = nullptr;
  auto out = std::unique_ptr<culi_results>(new (std::nothrow) culi_results);
  if (!out) return CULI_E_ARG;
  auto st = std::make_shared<SymTable>();
  Results& M = out->r;
  uint64_t total = 0;
  for (int k = 0; k < nranks; ++k) {
    if (sizes[k] < sizeof(ResHeader)) return CULI_E_ARG;
    ResHeader h;
    std::memcpy(&h, blobs[k], sizeof h);
    if (h.magic != RES_MAGIC) return CULI_E_ARG;
    total += h.nforms;
  }
  M.resize(total);
  std::fill(M.tag.begin(), M.tag.end(), (uint8_t)K_ERROR);
  std::fill(M.err.begin(), M.err.end(), (uint8_t)E_OOM);
  std::vector<char> seen(total, 0);
  for (int k = 0; k < nranks; ++k) {
    const char* p = (const char*)blobs[k];
    ResHeader h;
    std::memcpy(&h, p, sizeof h);
    size_t need = sizeof h + h.nforms * sizeof(RecWire) + h.npayload * sizeof(Token) + h.names_bytes +
                  h.nstr;
    if (sizes[k] < need) return CULI_E_ARG;
    const char* recp = p + sizeof h;
    const char* payp = recp + h.nforms * sizeof(RecWire);
    const char* namp = payp + h.npayload * sizeof(Token);
    const char* strp = namp + h.names_bytes;
    std::vector<uint32_t> remap;                      // rank symbol id -> merged id
    for (size_t q = 0; q < h.names_bytes;) {
      size_t e = q;
      while (e < h.names_bytes && namp[e]) ++e;
      remap.push_back(st->intern(namp + q, e - q));
      q = e + 1;
    }
    uint64_t pay_base = M.payload.size();
    uint64_t str_base = M.strings.size();
    M.strings.append(strp, h.nstr);
    auto fix = [&](uint32_t tag, uint64_t w) -> uint64_t {
      if (tag == K_SYM) return (uint64_t)remap.at((uint32_t)w);
      if (tag == K_STR) return pack2((uint32_t)(lo32h(w) + str_base), (uint32_t)(w >> 32));
      return w;
    };
    for (uint64_t t = 0; t < h.npayload; ++t) {
      Token tok;
      std::memcpy(&tok, payp + t * sizeof(Token), sizeof tok);
      tok.word = fix(tok.tag, tok.word);
      M.payload.push_back(tok);
    }
    for (uint64_t i = 0; i < h.nforms; ++i) {
      RecWire w;
      std::memcpy(&w, recp + i * sizeof w, sizeof w);
      uint32_t gi = form_index[k][i];
      if (gi >= total || seen[gi]) return CULI_E_ARG;
      seen[gi] = 1;
      uint64_t word = w.word;
      if (!w.err) {
        if (w.tag == K_CONS || w.tag == K_STR) word = pack2((uint32_t)(lo32h(word) + pay_base), (uint32_t)(word >> 32));
        else word = fix(w.tag, word);
      }
      M.tag[gi] = w.tag;
      M.err[gi] = w.err;
      M.steps[gi] = w.steps;
      M.word[gi] = word;
    }
  }
  M.syms = st;
  *merged = out.release();
  return CULI_OK;
}

}  // extern "C"

// ---- device-resident result gather (PAPER L584-589 ordered result assembly) ---------------
namespace {
constexpr uint64_t RES2_MAGIC = 0x32534552494c5543ull;   // "CULIRES2"
constexpr uint64_t EXP_PAYLOAD_CAP = 1, EXP_CTX_PAYLOAD = 2, EXP_FALLBACK = 4, EXP_OOM = 8;

struct Res2Header {
  uint64_t magic, nforms, npayload, names_bytes, nstr, paycap, overflow, pad;
};
static_assert(sizeof(Res2Header) == 64, "64-byte export header");

inline uint64_t align16(uint64_t x) { return (x + 15) & ~15ull; }

struct Res2Layout {
  uint64_t o_tag, o_err, o_steps, o_word, o_names, o_str, o_pay;
  Res2Layout(uint64_t n, uint64_t names, uint64_t nstr) {
    o_tag = sizeof(Res2Header);
    o_err = o_tag + n;
    o_steps = align8(o_err + n);
    o_word = o_steps + 8 * n;
    o_names = o_word + 8 * n;
    o_str = o_names + names;
    o_pay = align16(o_str + nstr);
  }
};

// header + payload tokens of an export, read on the device: no host synchronisation in the step
__global__ void export_pack_kernel(char* buf, Res2Header h, const unsigned long long* pcount, const uint4* payload,
                                   uint64_t o_pay, const int* flags, const uint32_t* nfallback) {
  unsigned long long pc = *pcount;
  uint64_t n = pc < h.paycap ? pc : h.paycap;
  uint4* out = reinterpret_cast<uint4*>(buf + o_pay);
  for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x)
    out[i] = payload[i];
  if (blockIdx.x == 0 && threadIdx.x == 0) {
    h.npayload = pc;
    h.overflow = (pc > h.paycap ? EXP_PAYLOAD_CAP : 0) | (flags[3] ? EXP_CTX_PAYLOAD : 0) |
                 (*nfallback ? EXP_FALLBACK : 0) | ((flags[0] || flags[4]) ? EXP_OOM : 0);
    *reinterpret_cast<Res2Header*>(buf) = h;
  }
}

// one rank of an import: scatter records by global form index, append payload tokens (offsets shifted,
// symbols re-interned through remap, string offsets shifted)
__global__ void import_rank_kernel(const char* buf, uint64_t n, uint64_t np, Res2Layout L, const uint32_t* fidx,
                                   uint32_t rank, uint32_t nranks, uint64_t total, const uint32_t* remap,
                                   uint32_t nremap, uint64_t pay_base, uint32_t str_base, uint8_t* mtag,
                                   uint8_t* merr, uint64_t* msteps, uint64_t* mword, uint4* mpay, int* bad) {
  uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  const uint8_t* tag = reinterpret_cast<const uint8_t*>(buf + L.o_tag);
  const uint8_t* err = reinterpret_cast<const uint8_t*>(buf + L.o_err);
  const uint64_t* steps = reinterpret_cast<const uint64_t*>(buf + L.o_steps);
  const uint64_t* word = reinterpret_cast<const uint64_t*>(buf + L.o_word);
  const uint4* pay = reinterpret_cast<const uint4*>(buf + L.o_pay);
  for (uint64_t k = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; k < n; k += stride) {
    uint64_t g = fidx ? fidx[k] : rank + k * nranks;
    if (g >= total) { atomicExch(bad, 1); continue; }
    uint32_t t = tag[k], e = err[k];
    uint64_t w = word[k];
    if (!e) {
      if (t == K_CONS || t == K_STR) w = pack2((uint32_t)((uint32_t)w + pay_base), (uint32_t)(w >> 32));
      else if (t == K_SYM) w = (uint32_t)w < nremap ? remap[(uint32_t)w] : (atomicExch(bad, 1), w);
    }
    mtag[g] = (uint8_t)t;
    merr[g] = (uint8_t)e;
    msteps[g] = steps[k];
    mword[g] = w;
  }
  for (uint64_t k = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; k < np; k += stride) {
    uint4 q = pay[k];
    if (q.z == K_SYM) {
      if (q.x < nremap) q.x = remap[q.x]; else atomicExch(bad, 1);
      q.y = 0;
    } else if (q.z == K_STR) {
      q.x += str_base;
    }
    mpay[pay_base + k] = q;
  }
}

template <typename T>
struct DevTmp {
  T* p = nullptr;
  ~DevTmp() { if (p) cudaFree(p); }
  cudaError_t alloc(size_t n) { return cudaMalloc(&p, std::max<size_t>(n, 1) * sizeof(T)); }
};
}  // namespace

extern "C" {

int culi_results_export(culi_ctx* c, void* dev_buf, size_t cap, size_t* bytes) {
  if (!c) return CULI_E_ARG;
  if (!c->have_batch) return CULI_E_STATE;
  uint64_t n = c->batch_forms;
  std::string names = names_blob(*c->syms);
  std::string strs = c->strings + c->batch_strings;
  Res2Layout L(n, names.size(), strs.size());
  if (!dev_buf) {
    unsigned long long pc = 0;
    CK(cudaMemcpyAsync(&pc, c->pcount, 8, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaStreamSynchronize(c->stream));
    if (bytes) *bytes = L.o_pay + 16 * pc;
    return CULI_OK;
  }
  if (cap < L.o_pay) {
    if (bytes) *bytes = L.o_pay;
    return CULI_E_ARG;
  }
  Res2Header h{};
  h.magic = RES2_MAGIC;
  h.nforms = n;
  h.names_bytes = names.size();
  h.nstr = strs.size();
  h.paycap = (cap - L.o_pay) / 16;
  if (bytes) *bytes = L.o_pay + 16 * h.paycap;
  char* d = (char*)dev_buf;
  if (n) {
    CK(cudaMemcpyAsync(d + L.o_tag, c->rtag.p, n, cudaMemcpyDeviceToDevice, c->stream));
    CK(cudaMemcpyAsync(d + L.o_err, c->rerr.p, n, cudaMemcpyDeviceToDevice, c->stream));
    CK(cudaMemcpyAsync(d + L.o_steps, c->rsteps.p, 8 * n, cudaMemcpyDeviceToDevice, c->stream));
    CK(cudaMemcpyAsync(d + L.o_word, c->rword.p, 8 * n, cudaMemcpyDeviceToDevice, c->stream));
  }
  // names and strings change only when the batch or the definitions do: a pageable H2D (staged before
  // the call returns, so the temporaries may go)
  std::string tail = names + strs;
  if (!tail.empty()) CK(cudaMemcpyAsync(d + L.o_names, tail.data(), tail.size(), cudaMemcpyHostToDevice, c->stream));
  unsigned blocks = (unsigned)std::min<uint64_t>((uint64_t)c->sms * 4, std::max<uint64_t>(1, (h.paycap + 255) / 256));
  export_pack_kernel<<<blocks, 256, 0, c->stream>>>(d, h, c->pcount, c->payload.p, L.o_pay, c->flags, c->nfallback);
  CK(cudaGetLastError());
  return CULI_OK;
}

int culi_results_import(culi_ctx* c, const void* const* bufs, const size_t* sizes, int nranks,
                        const uint32_t* const* form_index, culi_results** merged) {
  if (!c || !bufs || !sizes || !merged || nranks <= 0) return CULI_E_ARG;
  *merged = nullptr;
  std::vector<Res2Header> hs(nranks);
  for (int r = 0; r < nranks; ++r) {
    if (!bufs[r] || sizes[r] < sizeof(Res2Header)) return CULI_E_ARG;
    CK(cudaMemcpyAsync(&hs[r], bufs[r], sizeof(Res2Header), cudaMemcpyDeviceToHost, c->stream));
  }
  CK(cudaStreamSynchronize(c->stream));
  uint64_t total = 0, ptotal = 0;
  std::vector<Res2Layout> Ls;
  for (int r = 0; r < nranks; ++r) {
    const Res2Header& h = hs[r];
    if (h.magic != RES2_MAGIC || h.overflow) return CULI_E_ARG;
    Ls.emplace_back(h.nforms, h.names_bytes, h.nstr);
    if (Ls.back().o_pay + 16 * h.npayload > sizes[r]) return CULI_E_ARG;
    total += h.nforms;
    ptotal += h.npayload;
  }
  // names -> merged symbol table (ids of this ctx's table kept), strings concatenated
  auto out = std::unique_ptr<culi_results>(new (std::nothrow) culi_results);
  if (!out) return CULI_E_ARG;
  auto st = std::make_shared<SymTable>(*c->syms);
  Results& M = out->r;
  std::vector<std::vector<uint32_t>> remaps(nranks);
  std::vector<uint32_t> str_base(nranks);
  for (int r = 0; r < nranks; ++r) {
    std::string blob(hs[r].names_bytes + hs[r].nstr, '\0');
    if (!blob.empty())
      CK(cudaMemcpyAsync(&blob[0], (const char*)bufs[r] + Ls[r].o_names, blob.size(), cudaMemcpyDeviceToHost, c->stream));
    CK(cudaStreamSynchronize(c->stream));
    for (size_t q = 0; q < hs[r].names_bytes;) {
      size_t e = blob.find('\0', q);
      if (e == std::string::npos || e >= hs[r].names_bytes) return CULI_E_ARG;
      remaps[r].push_back(st->intern(blob.data() + q, e - q));
      q = e + 1;
    }
    str_base[r] = (uint32_t)M.strings.size();
    M.strings.append(blob, hs[r].names_bytes, hs[r].nstr);
  }
  if (form_index) {                                   // a permutation of [0, total) across the ranks
    std::vector<char> seen(total, 0);
    for (int r = 0; r < nranks; ++r) {
      if (!form_index[r] && hs[r].nforms) return CULI_E_ARG;
      for (uint64_t k = 0; k < hs[r].nforms; ++k) {
        uint32_t g = form_index[r][k];
        if (g >= total || seen[g]) return CULI_E_ARG;
        seen[g] = 1;
      }
    }
  } else {                                            // strided deal: rank r holds r, r + k, r + 2k ...
    for (int r = 0; r < nranks; ++r)
      if (hs[r].nforms != (total + nranks - 1 - r) / nranks) return CULI_E_ARG;
  }
  DevTmp<uint8_t> mtag, merr;
  DevTmp<uint64_t> msteps, mword;
  DevTmp<uint4> mpay;
  DevTmp<int> bad;
  CK(mtag.alloc(total));
  CK(merr.alloc(total));
  CK(msteps.alloc(total));
  CK(mword.alloc(total));
  CK(mpay.alloc(ptotal));
  CK(bad.alloc(1));
  CK(cudaMemsetAsync(bad.p, 0, sizeof(int), c->stream));
  std::vector<DevTmp<uint32_t>> dremap(nranks), dfidx(nranks);
  uint64_t pay_base = 0;
  for (int r = 0; r < nranks; ++r) {
    CK(dremap[r].alloc(remaps[r].size()));
    if (!remaps[r].empty())
      CK(cudaMemcpyAsync(dremap[r].p, remaps[r].data(), 4 * remaps[r].size(), cudaMemcpyHostToDevice, c->stream));
    const uint32_t* fi = nullptr;
    if (form_index && hs[r].nforms) {
      CK(dfidx[r].alloc(hs[r].nforms));
      CK(cudaMemcpyAsync(dfidx[r].p, form_index[r], 4 * hs[r].nforms, cudaMemcpyHostToDevice, c->stream));
      fi = dfidx[r].p;
    }
    uint64_t work = std::max(hs[r].nforms, hs[r].npayload);
    unsigned blocks = (unsigned)std::min<uint64_t>((uint64_t)c->sms * 8, std::max<uint64_t>(1, (work + 255) / 256));
    import_rank_kernel<<<blocks, 256, 0, c->stream>>>((const char*)bufs[r], hs[r].nforms, hs[r].npayload, Ls[r], fi,
                                                      (uint32_t)r, (uint32_t)nranks, total, dremap[r].p,
                                                      (uint32_t)remaps[r].size(), pay_base, str_base[r], mtag.p,
                                                      merr.p, msteps.p, mword.p, mpay.p, bad.p);
    CK(cudaGetLastError());
    pay_base += hs[r].npayload;
  }
  M.resize(total);
  M.payload.resize(ptotal);
  int hbad = 0;
  if (total) {
    CK(cudaMemcpyAsync(M.tag.data(), mtag.p, total, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaMemcpyAsync(M.err.data(), merr.p, total, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaMemcpyAsync(M.steps.data(), msteps.p, 8 * total, cudaMemcpyDeviceToHost, c->stream));
    CK(cudaMemcpyAsync(M.word.data(), mword.p, 8 * total, cudaMemcpyDeviceToHost, c->stream));
  }
  if (ptotal) CK(cudaMemcpyAsync(M.payload.data(), mpay.p, 16 * ptotal, cudaMemcpyDeviceToHost, c->stream));
  CK(cudaMemcpyAsync(&hbad, bad.p, sizeof hbad, cudaMemcpyDeviceToHost, c->stream));
  CK(cudaStreamSynchronize(c->stream));
  if (hbad) return CULI_E_ARG;
  M.syms = st;
  *merged = out.release();
  return CULI_OK;
}

}  // extern "C"
