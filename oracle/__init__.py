"""ctypes wrapper around the oracle (culi_oracle.cpp).  TEST INFRASTRUCTURE ONLY.

Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference legs may import
this package.  It shares no code with paper_conf_cluster_subdbn18_b200/ (the CUDA path).
"""
from __future__ import annotations

import ctypes
import dataclasses
import os
import subprocess

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "culi_oracle.cpp")
_LIB = os.path.join(_HERE, "liboracle.so")

ERR_NAMES = ["OK", "TYPE", "ARITY", "DIV0", "SYNTAX", "ARG", "DEPTH", "FUEL", "DEFINE_IN_BATCH", "OOM"]
DEFAULT_MAX_DEPTH = 1024
DEFAULT_FUEL = 1 << 40


def build(force: bool = False) -> str:
    """Compile the oracle with g++ (-ffp-contract=off: no FMA contraction, SURVEY c.9)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        subprocess.check_call(["g++", "-std=c++17", "-O2", "-ffp-contract=off", "-fPIC", "-shared",
                               "-pthread", "-o", _LIB, _SRC])
    return _LIB


_lib = None


def _load():
    global _lib
    if _lib is None:
        lib = ctypes.CDLL(build())
        lib.oracle_new.restype = ctypes.c_void_p
        lib.oracle_new.argtypes = [ctypes.c_uint32, ctypes.c_uint64]
        lib.oracle_delete.argtypes = [ctypes.c_void_p]
        lib.oracle_free.argtypes = [ctypes.c_void_p]
        lib.oracle_define.restype = ctypes.c_int
        lib.oracle_define.argtypes = [ctypes.c_void_p, ctypes.c_char_p, ctypes.c_size_t,
                                      ctypes.POINTER(ctypes.c_int64), ctypes.POINTER(ctypes.c_int),
                                      ctypes.POINTER(ctypes.c_size_t)]
        lib.oracle_eval.restype = ctypes.c_int
        lib.oracle_eval.argtypes = [ctypes.c_void_p, ctypes.c_char_p, ctypes.c_size_t, ctypes.c_int,
                                    ctypes.c_int, ctypes.POINTER(ctypes.c_void_p),
                                    ctypes.POINTER(ctypes.c_size_t), ctypes.POINTER(ctypes.c_double),
                                    ctypes.POINTER(ctypes.c_uint64), ctypes.POINTER(ctypes.c_uint64),
                                    ctypes.POINTER(ctypes.c_size_t)]
        lib.oracle_read_print.restype = ctypes.c_int
        lib.oracle_read_print.argtypes = [ctypes.c_void_p, ctypes.c_char_p, ctypes.c_size_t,
                                          ctypes.POINTER(ctypes.c_void_p),
                                          ctypes.POINTER(ctypes.c_size_t),
                                          ctypes.POINTER(ctypes.c_size_t)]
        _lib = lib
    return _lib


class OracleError(Exception):
    pass


@dataclasses.dataclass
class Result:
    err: int          # 0 = value, else error code (SURVEY c.10)
    steps: int        # canonical eval steps (c.4)
    printed: str      # printer output (c.8); "#<error NAME>" for errors

    @property
    def err_name(self) -> str:
        return ERR_NAMES[self.err]


@dataclasses.dataclass
class BatchRun:
    results: list
    seconds: float
    total_steps: int
    nforms: int


class Session:
    """One interpreter session: a global environment that persists across define/eval calls."""

    def __init__(self, max_depth: int = DEFAULT_MAX_DEPTH, fuel: int = DEFAULT_FUEL):
        self._lib = _load()
        self._s = self._lib.oracle_new(max_depth, fuel)

    def __del__(self):
        if getattr(self, "_s", None):
            self._lib.oracle_delete(self._s)
            self._s = None

    def define(self, text: str) -> None:
        b = text.encode()
        fi = ctypes.c_int64(-1)
        fe = ctypes.c_int(0)
        off = ctypes.c_size_t(0)
        rc = self._lib.oracle_define(self._s, b, len(b), ctypes.byref(fi), ctypes.byref(fe),
                                     ctypes.byref(off))
        if rc == -2:
            raise OracleError("read error at offset %d" % off.value)
        if rc != 0:
            raise OracleError("define failed at form %d: %s" % (fi.value, ERR_NAMES[fe.value]))

    def eval_batch(self, text: str, nthreads: int = 1, want_output: bool = True) -> BatchRun:
        b = text.encode()
        out = ctypes.c_void_p()
        out_len = ctypes.c_size_t(0)
        secs = ctypes.c_double(0)
        tot = ctypes.c_uint64(0)
        nf = ctypes.c_uint64(0)
        off = ctypes.c_size_t(0)
        rc = self._lib.oracle_eval(self._s, b, len(b), nthreads, 1 if want_output else 0,
                                   ctypes.byref(out), ctypes.byref(out_len), ctypes.byref(secs),
                                   ctypes.byref(tot), ctypes.byref(nf), ctypes.byref(off))
        if rc == -2:
            raise OracleError("read error at offset %d" % off.value)
        results = []
        if want_output:
            raw = ctypes.string_at(out.value, out_len.value).decode()
            self._lib.oracle_free(out)
            for line in raw.splitlines():
                e, s, p = line.split("\t", 2)
                results.append(Result(int(e), int(s), p))
        return BatchRun(results, secs.value, tot.value, nf.value)

    def eval(self, text: str) -> list:
        return self.eval_batch(text).results

    def eval1(self, text: str) -> Result:
        r = self.eval(text)
        assert len(r) == 1, r
        return r[0]

    def read_print(self, text: str) -> list:
        b = text.encode()
        out = ctypes.c_void_p()
        out_len = ctypes.c_size_t(0)
        off = ctypes.c_size_t(0)
        rc = self._lib.oracle_read_print(self._s, b, len(b), ctypes.byref(out), ctypes.byref(out_len),
                                         ctypes.byref(off))
        if rc == -2:
            raise OracleError("read error at offset %d" % off.value)
        raw = ctypes.string_at(out.value, out_len.value).decode()
        self._lib.oracle_free(out)
        return raw.splitlines()
