"""Builders for libculi's serialized-results wire format (culi_results_serialize), used by the CPU tests
of the gather/merge path.  Layout (csrc/culi_dist.cu):
  header  8 x u64  {magic "CULIRES1", nforms, npayload, names_bytes, nstr, 0, 0, 0}
  records nforms x {steps u64, word u64, tag u8, err u8, pad[6]}
  payload npayload x {word u64, tag u32, pad u32}        (pre-order tokens of list/string results)
  names   NUL-separated symbol names in id order
  strings raw bytes
"""
from __future__ import annotations

import struct

MAGIC = 0x31534552494C5543
RESERVED = ["quote", "if", "define", "defun", "defmacro", "lambda", "let", "progn", "setq",
            "quasiquote", "unquote", "unquote-splicing",
            "+", "-", "*", "/", "rem", "mod", "sqrt", "float", "trunc",
            "=", "<", ">", "<=", ">=", "eq", "equal", "null", "not",
            "atom", "consp", "numberp", "symbolp", "cons", "car", "cdr", "list",
            "length", "append", "reverse", "nth", "|||"]
NIL, T, INT, FLOAT, STR, SYM, CONS = 0, 1, 2, 3, 4, 5, 6


def blob(records, payload=(), names=(), strings=b""):
    """records: (tag, err, steps, word); payload: (tag, word); names: extra symbols after RESERVED."""
    allnames = RESERVED + list(names)
    nb = b"".join(n.encode() + b"\0" for n in allnames)
    out = struct.pack("<8Q", MAGIC, len(records), len(payload), len(nb), len(strings), 0, 0, 0)
    for tag, err, steps, word in records:
        out += struct.pack("<QQBB6x", steps, word & (2**64 - 1), tag, err)
    for tag, word in payload:
        out += struct.pack("<QII", word & (2**64 - 1), tag, 0)
    return out + nb + strings


def sym_id(name, extra):
    return (RESERVED + list(extra)).index(name)
