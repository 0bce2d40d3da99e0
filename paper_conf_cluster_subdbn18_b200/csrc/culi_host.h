// culi_host.h — host-side structures of libculi.so: symbol table, node image, results.
#pragma once
#include <cstddef>
#include <cstdint>
#include <memory>
#include <string>
#include <unordered_map>
#include <utility>
#include <vector>

#include "culi_internal.h"

namespace culi {

// Dense symbol interning (north_star: "symbol interning").  Reserved names take ids [0, N_RESERVED).
struct SymTable {
  std::unordered_map<std::string, uint32_t> ids;
  std::vector<std::string> names;
  SymTable();
  uint32_t intern(const char* s, size_t n);
};

extern const char* const kSpecialName[N_SPECIALS];
extern const char* const kBuiltinName[N_BUILTINS];
extern const char* const kErrName[10];

// A compact, relocatable node image produced by the host reader.  Local numbering:
// 0 = nil, 1 = T, node k of the image at local index IMG_FIRST + k.  Cons words hold local indices;
// string words hold offsets into `strings`.
struct Image {
  std::vector<uint8_t> tag;
  std::vector<uint64_t> word;
  std::vector<uint32_t> roots;     // local index of each top-level form
  std::string strings;
  uint32_t max_sym = 0;            // largest symbol id referenced + 1
  std::vector<uint32_t> wide_len;  // pairs (local index of a wide list's second cell, cells from it to the end)
};

// Returns 0 or CULI_E_PARSE with *err_offset.
int read_image(SymTable& st, const char* text, size_t len, Image& out, size_t* err_offset);

// Result of one form as copied back from the device.
struct Record {
  uint8_t tag;      // Kind (K_ERROR when err != 0)
  uint8_t err;
  uint64_t steps;
  uint64_t word;    // INT/FLOAT/SYM payload, BUILTIN/SPECIAL op, or payload offset|len<<32 for CONS/STR
};

// Serialized value token (pre-order; CONS is followed by its car then its cdr).
struct Token {
  uint64_t word;
  uint32_t tag;
  uint32_t pad;
};

// Host memory for result arrays: large blocks come from a process-wide cache of page-locked blocks (so the
// device -> host copies of a fetch run at DMA speed and repeated fetches neither re-pin nor page-fault),
// and elements are default-initialised (a fetch overwrites them; no zero fill).  culi_host.cpp.
void* pinned_pool_alloc(size_t bytes);
void pinned_pool_free(void* p, size_t bytes);
template <typename T>
struct ResultAlloc {
  using value_type = T;
  ResultAlloc() = default;
  template <typename U>
  ResultAlloc(const ResultAlloc<U>&) {}
  T* allocate(size_t n) { return static_cast<T*>(pinned_pool_alloc(n * sizeof(T))); }
  void deallocate(T* p, size_t n) { pinned_pool_free(p, n * sizeof(T)); }
  template <typename U>
  void construct(U* p) { ::new (static_cast<void*>(p)) U; }   // default-init: no zeroing
  template <typename U, typename... A>
  void construct(U* p, A&&... a) { ::new (static_cast<void*>(p)) U(std::forward<A>(a)...); }
  template <typename U>
  bool operator==(const ResultAlloc<U>&) const { return true; }
  template <typename U>
  bool operator!=(const ResultAlloc<U>&) const { return false; }
};
template <typename T>
using rvec = std::vector<T, ResultAlloc<T>>;

struct Results {
  // records as structure of arrays, so the device arrays are copied straight in (no per-record work)
  rvec<uint8_t> tag, err;
  rvec<uint64_t> steps, word;
  size_t size() const { return tag.size(); }
  Record at(size_t i) const { return Record{tag[i], err[i], steps[i], word[i]}; }
  void resize(size_t n) { tag.resize(n); err.resize(n); steps.resize(n); word.resize(n); }
  rvec<Token> payload;
  std::shared_ptr<const SymTable> syms;   // names for SYM tokens
  std::string strings;                    // bytes for STR tokens
  void print(uint32_t i, std::string& out) const;
  void print_token_range(size_t& pos, std::string& out) const;
};

void print_float(double d, std::string& out);

}  // namespace culi
