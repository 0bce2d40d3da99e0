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
  uint64_t o_tag, o_word, o_gtag, o_gword, o_str, o_names, total;
  EnvLayout(const EnvHeader& h) {
    o_tag = sizeof(EnvHeader);
    o_word = align8(o_tag + h.mark);
    o_gtag = o_word + 8 * h.mark;
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
  CK(cudaMemcpyAsync(d + L.o_tag, c->H.tag, h.mark, cudaMemcpyDeviceToDevice, c->stream));
  CK(cudaMemcpyAsync(d + L.o_word, c->H.word, 8 * h.mark, cudaMemcpyDeviceToDevice, c->stream));
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
  CK(cudaMemcpyAsync(c->H.tag, d + L.o_tag, h.mark, cudaMemcpyDeviceToDevice, c->stream));
  CK(cudaMemcpyAsync(c->H.word, d + L.o_word, 8 * h.mark, cudaMemcpyDeviceToDevice, c->stream));
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
