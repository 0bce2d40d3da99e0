// culi_reader.h — device reader declarations shared by culi_reader.cu and culi_capi.cu.
#pragma once
#include <stdint.h>

#include <string>

struct culi_ctx;

namespace culi {

constexpr uint32_t ROOT = 0xffffffffu;           // parent of a top-level datum

// Device symbol table (culi_reader.cu intern): open addressing over 64-bit name hashes.
struct DevSyms {
  uint64_t* key = nullptr;       // slot -> name hash (0 = empty)
  uint32_t* id = nullptr;        // slot -> symbol id (0xffffffff = being published)
  uint64_t* tag = nullptr;       // slot -> first 7 name bytes | min(length, 255) << 56
  uint64_t* noff = nullptr;      // id -> pool offset | length << 32
  uint8_t* pool = nullptr;       // name bytes
  uint32_t* count = nullptr;     // [0] next id, [2..3] pool top (u64), [4] overflow
  uint32_t cap = 0;              // slots (power of two)
  uint32_t idcap = 0;
  uint64_t pool_cap = 0;
};

// Summary of one read, written by the reader kernels.
struct ReadInfo {
  unsigned long long err_pos;    // smallest offending byte offset (~0 = none)
  unsigned long long open_pos;   // 1 + offset of the innermost '(' still open at the end
  unsigned long long str_pos;    // 1 + offset of the last string start
  uint32_t max_key;              // deepest list + 1
  uint32_t nstr;                 // string literals
  int final_depth;
  uint32_t last_kind;
  uint32_t last_pos;
  uint32_t nforms;
  uint32_t flags;                // RF_*
  uint32_t nvalid;               // lists queued for special-form syntax validation
};
constexpr uint32_t RF_PAR_ROOT_HEAD = 1;         // some top-level form is (||| ...)
constexpr uint32_t RF_PAR_NESTED = 2;            // ||| is the car of some other cell
constexpr uint32_t RF_WIDE = 4;                  // some top-level form has >= WIDE_MIN arguments
constexpr uint32_t RF_SETQ = 8;                  // the setq symbol occurs (R7)
constexpr uint32_t RF_CLOSURE = 16;              // lambda or defun occurs: closures may exist
constexpr uint32_t RF_WIDE_NESTED = 32;          // a list below the top level, not a quote's operand, has
                                                 // >= WIDE_MIN elements after its head (NEST_EVAL)

struct ReadOut {
  uint32_t nforms = 0;
  uint32_t nodes = 0;
  std::string strings;           // the batch's string bytes (host mirror, for printing)
  bool par_root_head = false, par_nested = false, wide = false, setq = false, closure = false;
  bool wide_nested = false;
};

// Parse `len` bytes (host or device pointer) into the heap at ctx->mark, the form table into ctx->roots
// and the wide-form table into ctx->wide.  CULI_E_PARSE sets *err_offset as culi_read does.
int device_read(culi_ctx* c, const char* text, size_t len, bool on_device, ReadOut* out, size_t* err_offset);

}  // namespace culi
