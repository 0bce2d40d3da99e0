// culi_host.cpp — host reader (text -> relocatable node image) and host printer of libculi.so.
//
// The paper reads on the device (§III-B.b) and names parsing the dominant GPU phase
// (L785-788); north_star moves the read to the host ("host reads into a compact node array") so the
// device runs only eval.  The reader is an iterative scanner (no recursion: inputs may nest deeply or
// hold a 1M-element list) that allocates every list spine as consecutive cells (SURVEY c.14), so the
// device's ||| fan-out can index list elements in O(1).
#include <cerrno>
#include <charconv>
#include <cmath>
#include <cstdlib>
#include <cstring>
#include <map>
#include <mutex>
#include <unordered_map>

#include <cuda_runtime.h>

#include "../../include/culi.h"
#include "culi_host.h"

namespace culi {

// ---- page-locked block cache for result arrays (culi_host.h ResultAlloc) --------------------------------
namespace {
constexpr size_t PIN_MIN = 1u << 20;             // smaller arrays: plain heap
constexpr size_t PIN_CACHE_MAX = 8ull << 30;     // cached (free) pinned bytes kept at most
struct PinCache {
  std::mutex mu;
  std::multimap<size_t, void*> free_blocks;      // capacity -> block
  std::unordered_map<void*, size_t> cap;         // block -> capacity (pinned blocks only)
  size_t cached = 0;
};
PinCache& pin_cache() {
  static PinCache* c = new PinCache;             // never destroyed: frees may run at exit
  return *c;
}
}  // namespace

void* pinned_pool_alloc(size_t bytes) {
  if (bytes < PIN_MIN) return ::operator new(bytes ? bytes : 1);
  PinCache& C = pin_cache();
  {
    std::lock_guard<std::mutex> g(C.mu);
    auto it = C.free_blocks.lower_bound(bytes);
    if (it != C.free_blocks.end() && it->first <= 2 * bytes) {
      void* p = it->second;
      C.cached -= it->first;
      C.free_blocks.erase(it);
      return p;
    }
  }
  size_t cap = size_t(1) << (64 - __builtin_clzll(bytes - 1));   // next power of two
  void* p = nullptr;
  if (cudaHostAlloc(&p, cap, cudaHostAllocDefault) != cudaSuccess) {
    cudaGetLastError();
    return ::operator new(bytes);                // no device / no pinned memory: plain heap
  }
  std::lock_guard<std::mutex> g(C.mu);
  C.cap[p] = cap;
  return p;
}

void pinned_pool_free(void* p, size_t bytes) {
  if (!p) return;
  if (bytes < PIN_MIN) { ::operator delete(p); return; }
  PinCache& C = pin_cache();
  std::lock_guard<std::mutex> g(C.mu);
  auto it = C.cap.find(p);
  if (it == C.cap.end()) { ::operator delete(p); return; }
  if (C.cached + it->second > PIN_CACHE_MAX) {
    C.cap.erase(it);
    cudaFreeHost(p);
    return;
  }
  C.cached += it->second;
  C.free_blocks.emplace(it->second, p);
}

const char* const kSpecialName[N_SPECIALS] = {"quote", "if", "define", "defun", "defmacro", "lambda",
                                              "let", "progn", "setq", "quasiquote", "unquote",
                                              "unquote-splicing"};
const char* const kBuiltinName[N_BUILTINS] = {
    "+", "-", "*", "/", "rem", "mod", "sqrt", "float", "trunc",
    "=", "<", ">", "<=", ">=", "eq", "equal", "null", "not",
    "atom", "consp", "numberp", "symbolp", "cons", "car", "cdr", "list",
    "length", "append", "reverse", "nth", "|||"};
const char* const kErrName[10] = {"NONE", "TYPE", "ARITY", "DIV0", "SYNTAX", "ARG", "DEPTH", "FUEL",
                                  "DEFINE_IN_BATCH", "OOM"};

SymTable::SymTable() {
  for (uint32_t k = 0; k < N_SPECIALS; ++k) intern(kSpecialName[k], std::strlen(kSpecialName[k]));
  for (uint32_t k = 0; k < N_BUILTINS; ++k) intern(kBuiltinName[k], std::strlen(kBuiltinName[k]));
}

uint32_t SymTable::intern(const char* s, size_t n) {
  std::string key(s, n);
  auto it = ids.find(key);
  if (it != ids.end()) return it->second;
  uint32_t id = (uint32_t)names.size();
  names.push_back(key);
  ids.emplace(std::move(key), id);
  return id;
}

// ---- token classification (SURVEY c.1, c.13 #2) -------------------------------------------------------
static inline bool is_space(char c) {
  return c == ' ' || c == '\t' || c == '\n' || c == '\r' || c == '\f' || c == '\v';
}
static inline bool is_digit(char c) { return c >= '0' && c <= '9'; }

// ^[+-]?[0-9]+$
static bool classify_int(const char* s, size_t n) {
  size_t i = (n > 0 && (s[0] == '+' || s[0] == '-')) ? 1 : 0;
  if (i == n) return false;
  for (; i < n; ++i)
    if (!is_digit(s[i])) return false;
  return true;
}

// ^[+-]?([0-9]+\.[0-9]*|\.[0-9]+)([eE][+-]?[0-9]+)?$ | ^[+-]?[0-9]+[eE][+-]?[0-9]+$
static bool classify_float(const char* s, size_t n) {
  size_t i = (n > 0 && (s[0] == '+' || s[0] == '-')) ? 1 : 0;
  size_t int_digits = 0, frac_digits = 0;
  bool dot = false;
  while (i < n && is_digit(s[i])) { ++i; ++int_digits; }
  if (i < n && s[i] == '.') {
    dot = true;
    ++i;
    while (i < n && is_digit(s[i])) { ++i; ++frac_digits; }
  }
  if (int_digits + frac_digits == 0) return false;
  bool expo = false;
  if (i < n && (s[i] == 'e' || s[i] == 'E')) {
    ++i;
    if (i < n && (s[i] == '+' || s[i] == '-')) ++i;
    size_t ed = 0;
    while (i < n && is_digit(s[i])) { ++i; ++ed; }
    if (ed == 0) return false;
    expo = true;
  }
  if (i != n) return false;
  return dot || expo;
}

namespace {
struct Open {
  bool quote;                  // a pending prefix (' ` ,) that completes after one datum
  size_t offset;               // byte offset of '(' or the prefix
  std::vector<uint32_t> elems; // elements of an open list
  uint32_t prefix_sym = SP_QUOTE;   // quote / quasiquote / unquote (reading R8)
};

struct Builder {
  SymTable& st;
  Image& img;
  std::vector<uint32_t> sym_node;   // per-image dedupe: symbol id -> local node (0 = none yet)

  uint32_t node(uint8_t tag, uint64_t word) {
    uint32_t idx = IMG_FIRST + (uint32_t)img.tag.size();
    img.tag.push_back(tag);
    img.word.push_back(word);
    return idx;
  }
  uint32_t symbol(uint32_t id) {
    if (id >= sym_node.size()) sym_node.resize(id + 1, 0);
    if (!sym_node[id]) sym_node[id] = node(K_SYM, id);
    if (id + 1 > img.max_sym) img.max_sym = id + 1;
    return sym_node[id];
  }
  // contiguous spine for a proper list (SURVEY c.14)
  uint32_t spine(const std::vector<uint32_t>& xs) {
    if (xs.empty()) return 0;
    uint32_t first = IMG_FIRST + (uint32_t)img.tag.size();
    uint32_t n = (uint32_t)xs.size();
    uint8_t valid = special_form_valid(xs) ? TAG_VALID : 0;
    for (uint32_t k = 0; k < n; ++k)
      node((uint8_t)(K_CONS | TAG_PROPER | (k == 0 ? valid : 0)), pack2(xs[k], k + 1 < n ? first + k + 1 : 0));
    if (n >= WIDE_LEN_MIN + 1) {                       // the device marks the second cell (TAG_LEN)
      img.wide_len.push_back(first + 1);
      img.wide_len.push_back(n - 1);
    }
    return first;
  }

  // ---- syntax of special forms (SURVEY c.5), checked once at read time -----------------------------
  uint32_t ltag(uint32_t L) const { return L < IMG_FIRST ? (L == 0 ? K_NIL : K_T) : img.tag[L - IMG_FIRST]; }
  uint64_t lword(uint32_t L) const { return L < IMG_FIRST ? 0 : img.word[L - IMG_FIRST]; }
  bool bindable(uint32_t L) const { return (ltag(L) & KIND_MASK) == K_SYM && lword(L) >= N_RESERVED; }
  std::vector<uint32_t> elems(uint32_t L) const {           // reader lists are proper
    std::vector<uint32_t> out;
    while (L != 0) { uint64_t w = lword(L); out.push_back((uint32_t)w); L = (uint32_t)(w >> 32); }
    return out;
  }
  bool is_list(uint32_t L) const { return L == 0 || (ltag(L) & KIND_MASK) == K_CONS; }
  bool params_ok(uint32_t L) const {
    if (!is_list(L)) return false;
    for (uint32_t p : elems(L)) if (!bindable(p)) return false;
    return true;
  }
  bool special_form_valid(const std::vector<uint32_t>& xs) const {
    uint32_t h = xs[0];
    if ((ltag(h) & KIND_MASK) != K_SYM || lword(h) >= N_SPECIALS) return false;
    size_t n = xs.size() - 1;
    switch (lword(h)) {
      case SP_QUOTE:
      case SP_QUASIQUOTE: return n == 1;
      case SP_IF: return n == 2 || n == 3;
      case SP_PROGN: return true;
      case SP_LAMBDA: return n >= 1 && params_ok(xs[1]);
      case SP_DEFINE:
      case SP_SETQ: return n == 2 && bindable(xs[1]);
      case SP_DEFUN:
      case SP_DEFMACRO: return n >= 2 && bindable(xs[1]) && params_ok(xs[2]);
      case SP_LET: {
        if (n < 1 || !is_list(xs[1])) return false;
        for (uint32_t b : elems(xs[1])) {
          if ((ltag(b) & KIND_MASK) != K_CONS) return false;
          std::vector<uint32_t> se = elems(b);
          if (se.size() != 2 || !bindable(se[0])) return false;
        }
        return true;
      }
    }
    return false;
  }
};
}  // namespace

int read_image(SymTable& st, const char* text, size_t len, Image& img, size_t* err_offset) {
  Builder B{st, img, {}};
  std::vector<Open> stack;
  size_t p = 0;
  auto fail = [&](size_t off) {
    if (err_offset) *err_offset = off;
    return (int)CULI_E_PARSE;
  };

  // deliver a finished datum to the innermost open construct
  auto deliver = [&](uint32_t d) {
    for (;;) {
      if (stack.empty()) { img.roots.push_back(d); return; }
      Open& top = stack.back();
      if (!top.quote) { top.elems.push_back(d); return; }
      uint32_t sym = top.prefix_sym;
      stack.pop_back();                              // 'x == (quote x), `x, ,x (R8)
      std::vector<uint32_t> q{B.symbol(sym), d};
      d = B.spine(q);
    }
  };

  for (;;) {
    while (p < len) {                                // whitespace and ; comments
      if (is_space(text[p])) { ++p; continue; }
      if (text[p] == ';') { while (p < len && text[p] != '\n') ++p; continue; }
      break;
    }
    if (p >= len) break;
    char c = text[p];
    if (c == '(') {
      stack.push_back(Open{false, p, {}});
      ++p;
    } else if (c == ')') {
      if (stack.empty() || stack.back().quote) return fail(p);
      std::vector<uint32_t> xs = std::move(stack.back().elems);
      stack.pop_back();
      ++p;
      deliver(B.spine(xs));
    } else if (c == '\'' || c == '`' || c == ',') {
      stack.push_back(Open{true, p, {}, c == '\'' ? (uint32_t)SP_QUOTE : c == '`' ? (uint32_t)SP_QUASIQUOTE
                                                                            : (uint32_t)SP_UNQUOTE});
      ++p;
    } else if (c == '"') {
      const void* q = std::memchr(text + p + 1, '"', len - p - 1);
      if (!q) return fail(p);
      size_t e = (const char*)q - text;
      uint64_t off = img.strings.size();
      img.strings.append(text + p + 1, e - p - 1);
      deliver(B.node(K_STR, pack2((uint32_t)off, (uint32_t)(e - p - 1))));
      p = e + 1;
    } else {
      size_t s = p;
      while (p < len && !is_space(text[p]) && text[p] != '(' && text[p] != ')') ++p;
      const char* t = text + s;
      size_t n = p - s;
      uint32_t d;
      if (n == 3 && std::memcmp(t, "nil", 3) == 0) {
        d = 0;
      } else if (n == 1 && t[0] == 'T') {
        d = 1;
      } else if (classify_int(t, n)) {
        std::string tok(t, n);
        errno = 0;
        long long v = std::strtoll(tok.c_str(), nullptr, 10);
        if (errno == ERANGE) return fail(s);
        d = B.node(K_INT, (uint64_t)v);
      } else if (classify_float(t, n)) {
        std::string tok(t, n);
        double v = std::strtod(tok.c_str(), nullptr);
        uint64_t bits;
        std::memcpy(&bits, &v, 8);
        d = B.node(K_FLOAT, bits);
      } else {
        d = B.symbol(st.intern(t, n));
      }
      deliver(d);
    }
  }
  if (!stack.empty()) return fail(stack.back().offset);
  return CULI_OK;
}

// ---- printer (§III-B.d; SURVEY c.8) ------------------------------------------------------
void print_float(double d, std::string& out) {
  if (std::isnan(d)) { out += "nan"; return; }
  if (std::isinf(d)) { out += d < 0 ? "-inf" : "inf"; return; }
  char buf[64];
  auto r = std::to_chars(buf, buf + sizeof buf, d);
  bool has = false;
  for (char* q = buf; q < r.ptr; ++q)
    if (*q == '.' || *q == 'e') has = true;
  out.append(buf, r.ptr);
  if (!has) out += ".0";
}

static void print_atom(const Results& R, uint32_t tag, uint64_t w, std::string& out) {
  switch (tag) {
    case K_NIL: out += "nil"; break;
    case K_T: out += "T"; break;
    case K_INT: out += std::to_string((long long)(int64_t)w); break;
    case K_FLOAT: { double d; std::memcpy(&d, &w, 8); print_float(d, out); break; }
    case K_SYM: out += R.syms->names[(uint32_t)w]; break;
    case K_STR:
      out += '"';
      out.append(R.strings, (uint32_t)w, (uint32_t)(w >> 32));
      out += '"';
      break;
    case K_BUILTIN: out += "#<builtin "; out += kBuiltinName[w]; out += '>'; break;
    case K_SPECIAL: out += "#<special "; out += kSpecialName[w]; out += '>'; break;
    case K_CLOSURE: out += "#<lambda>"; break;
    case K_MACRO: out += "#<macro>"; break;
    default: out += "#<?>"; break;
  }
}

void Results::print_token_range(size_t& pos, std::string& out) const {
  const Token& t = payload[pos++];
  if (t.tag != K_CONS) { print_atom(*this, t.tag, t.word, out); return; }
  out += '(';
  print_token_range(pos, out);                        // car
  for (;;) {                                          // cdr chain iteratively
    const Token& n = payload[pos];
    if (n.tag == K_CONS) { ++pos; out += ' '; print_token_range(pos, out); continue; }
    ++pos;
    if (n.tag != K_NIL) { out += " . "; print_atom(*this, n.tag, n.word, out); }
    break;
  }
  out += ')';
}

void Results::print(uint32_t i, std::string& out) const {
  const Record r = at(i);
  if (r.err) { out += "#<error "; out += kErrName[r.err < 10 ? r.err : 9]; out += '>'; return; }
  if (r.tag == K_CONS || r.tag == K_STR) {
    size_t pos = (uint32_t)r.word;
    print_token_range(pos, out);
    return;
  }
  print_atom(*this, r.tag, r.word, out);
}

}  // namespace culi
