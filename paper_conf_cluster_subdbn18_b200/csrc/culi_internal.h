// culi_internal.h — internal layout shared by the host reader/printer and the device kernels of
// libculi.so.  (Product code: never included by oracle/.)
//
// Heap: node pool in HBM (§III-A.c "nodes are stored in a large array ... the sequentially
// next free node"; node = value + links, L288-293 §III-A.a Fig.1), 16 bytes per node (struct Node):
//   tag     : uint8   kind (low 4 bits) | CULI_TAG_PROPER (cons whose cdr chain ends in nil)
//   word    : uint64  payload — INT int64 / FLOAT f64 bits / SYM id / STR off|len<<32 /
//                     CONS car|cdr<<32 (node indices) / BUILTIN,SPECIAL op /
//                     CLOSURE,MACRO code|env<<32 (code = cons (params . body), env = heap frame or 0) /
//                     FRAME parent|n<<32 / BIND sym|valnode<<32
// Node 0 is nil, node 1 is T.  Heap frames are 1 FRAME node + n BIND nodes + n value slots.
#pragma once
#include <stdint.h>

namespace culi {

enum Kind : uint8_t {
  K_NIL = 0, K_T = 1, K_INT = 2, K_FLOAT = 3, K_STR = 4, K_SYM = 5, K_CONS = 6, K_BUILTIN = 7,
  K_SPECIAL = 8, K_CLOSURE = 9, K_MACRO = 10, K_FRAME = 11, K_BIND = 12, K_ERROR = 13,
  K_UNBOUND = 15
};
constexpr uint8_t TAG_PROPER = 0x10;
// Set by the host reader on a list whose head is a special-form name (always the special form: the
// names are reserved, c.5) and whose syntax it has already validated per c.5; the device skips the
// checks for such lists.  Lists built at run time (macro expansions) never carry it.
constexpr uint8_t TAG_VALID = 0x20;
// Set by the readers on the second cell of a list with at least WIDE_MIN + 1 cells, whose `len` field
// (struct Node) then holds the number of cells from it to the end of the list: a wide data list / (list ...)
// starts its element count there (culi_machine.cuh DATA_START) in O(1) instead of walking the spine.  Any
// write of a tag byte clears it, so a cell built at run time never carries a stale length.
constexpr uint8_t TAG_LEN = 0x40;
constexpr uint32_t WIDE_LEN_MIN = 64;   // == WIDE_MIN (culi_eval.cuh)
constexpr uint8_t K_AUX = 14;    // second node of a closure/macro: nparams | first param symbol << 32
constexpr uint8_t KIND_MASK = 0x0f;

enum ErrCode : uint8_t {
  E_NONE = 0, E_TYPE = 1, E_ARITY = 2, E_DIV0 = 3, E_SYNTAX = 4, E_ARG = 5, E_DEPTH = 6, E_FUEL = 7,
  E_DEFINE_IN_BATCH = 8, E_OOM = 9
};

// Reserved symbols (SURVEY c.5 "reserved names"): ids [0, N_RESERVED) in this order.
enum SpecialOp : uint8_t { SP_QUOTE, SP_IF, SP_DEFINE, SP_DEFUN, SP_DEFMACRO, SP_LAMBDA, SP_LET,
                           SP_PROGN, SP_SETQ, SP_QUASIQUOTE, SP_UNQUOTE, SP_UNQUOTE_SPLICING, N_SPECIALS };
enum BuiltinOp : uint8_t {
  BI_ADD, BI_SUB, BI_MUL, BI_DIV, BI_REM, BI_MOD, BI_SQRT, BI_FLOAT, BI_TRUNC,
  BI_NUMEQ, BI_LT, BI_GT, BI_LE, BI_GE, BI_EQ, BI_EQUAL, BI_NULL, BI_NOT,
  BI_ATOM, BI_CONSP, BI_NUMBERP, BI_SYMBOLP, BI_CONS, BI_CAR, BI_CDR, BI_LIST,
  BI_LENGTH, BI_APPEND, BI_REVERSE, BI_NTH, BI_PAR, N_BUILTINS
};
constexpr uint32_t N_RESERVED = N_SPECIALS + N_BUILTINS;

// Image-local node numbering: 0 = nil, 1 = T, image node k at local index 2 + k.  Relocation maps local
// index L >= 2 to heap index base + (L - 2).
constexpr uint32_t IMG_FIRST = 2;

#ifdef __CUDACC__
#define CULI_HD __host__ __device__ __forceinline__
#else
#define CULI_HD inline
#endif
CULI_HD uint64_t pack2(uint32_t lo, uint32_t hi) { return (uint64_t)lo | ((uint64_t)hi << 32); }

// Device heap node: payload and tag co-located in 16 bytes, so the device reads a node with one aligned
// 16-byte load (north_star "coalesced, vectorised node loads"; culi_machine.cuh ldnode).  TagArr / WordArr
// view the node array as the tag[] / word[] arrays the kernels index (node i's fields, 16 bytes apart).
// Host images stay structure-of-arrays (9 B/node on the wire); the relocate kernel interleaves them.
struct alignas(16) Node {
  uint64_t word;
  uint8_t tag;
  uint8_t pad[3];
  uint32_t len;                // TAG_LEN cells: cells from here to the end of the list
};
static_assert(sizeof(Node) == 16, "one 16-byte access per node");
struct TagArr {
  Node* p;
  CULI_HD uint8_t& operator[](uint64_t i) const { return p[i].tag; }
  CULI_HD TagArr operator+(uint64_t o) const { return TagArr{p + o}; }
};
struct WordArr {
  Node* p;
  CULI_HD uint64_t& operator[](uint64_t i) const { return p[i].word; }
  CULI_HD WordArr operator+(uint64_t o) const { return WordArr{p + o}; }
};

}  // namespace culi
