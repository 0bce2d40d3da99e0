"""Thin ctypes binding of libculi.so (include/culi.h): argument marshalling only.

Every step of read/define/eval runs in libculi.so (host reader in C++, eval in sm_100a CUDA kernels).
There is no Python or CPU fallback: if libculi.so is missing or no CUDA device is visible, the calls
raise.  The raw C entry points are exported under their C names (culi_init, culi_read, ...); `Context`
is a convenience wrapper over them.
"""
from __future__ import annotations

import ctypes
import os

HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("CULI_LIB") or os.path.join(HERE, "libculi.so")   # CULI_LIB: A/B builds (tools/)

ERR_NAMES = ["NONE", "TYPE", "ARITY", "DIV0", "SYNTAX", "ARG", "DEPTH", "FUEL", "DEFINE_IN_BATCH", "OOM"]
TAG_NAMES = {0: "NIL", 1: "T", 2: "INT", 3: "FLOAT", 4: "STRING", 5: "SYMBOL", 6: "CONS", 7: "BUILTIN",
             8: "SPECIAL", 9: "CLOSURE", 10: "MACRO", 13: "ERROR"}

CULI_F_NO_BINNING = 1
CULI_F_NO_FANOUT = 2
CULI_F_NO_STAGING = 4
CULI_F_NO_VOTING = 8
CULI_F_NO_NESTED = 16
CULI_F_NO_SPLIT = 32
CULI_F_NO_GC = 64
CULI_F_NO_GRAPH = 128
CULI_F_DEVICE_READ = 256

SYMBOLS = [
    "culi_default_opts", "culi_init", "culi_shutdown", "culi_read", "culi_image_nforms",
    "culi_image_nnodes", "culi_image_free", "culi_define", "culi_eval_batch", "culi_upload",
    "culi_eval_uploaded", "culi_fetch_results", "culi_release", "culi_results_count", "culi_result_info",
    "culi_result_int", "culi_result_float", "culi_print", "culi_results_totals", "culi_results_free",
    "culi_env_export", "culi_env_import", "culi_results_serialize", "culi_results_merge",
    "culi_status_string", "culi_error_name", "culi_last_timing", "culi_records_device",
    "culi_last_stats", "culi_last_splits", "culi_last_split_claims", "culi_last_waits", "culi_last_reruns", "culi_image_pin", "culi_results_wire_bytes",
    "culi_define_text", "culi_eval_text", "culi_upload_text", "culi_last_read", "culi_collect",
    "culi_heap_usage", "culi_arena_bytes", "culi_eval_batch_async", "culi_sync", "culi_complete",
    "culi_results_export", "culi_results_import",
]


class CuliError(RuntimeError):
    def __init__(self, status: int, what: str):
        self.status = status
        super().__init__("%s failed: %s (%d)" % (what, _status_string(status), status))


class culi_opts(ctypes.Structure):
    _fields_ = [("device", ctypes.c_int), ("stream", ctypes.c_void_p), ("heap_nodes", ctypes.c_uint64),
                ("max_depth", ctypes.c_uint32), ("fuel", ctypes.c_uint64),
                ("vstack_entries", ctypes.c_uint32), ("slots", ctypes.c_uint32), ("flags", ctypes.c_uint32),
                ("heap_base", ctypes.c_void_p), ("heap_bytes", ctypes.c_uint64)]


_lib = None


def load(path: str = LIB_PATH) -> ctypes.CDLL:
    """Load libculi.so; raises (never falls back) if it is missing."""
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(path):
        raise ImportError("libculi.so not built (%s); run __graft_entry__.build()" % path)
    L = ctypes.CDLL(path)
    P, U32, U64, SZ, I = ctypes.c_void_p, ctypes.c_uint32, ctypes.c_uint64, ctypes.c_size_t, ctypes.c_int
    pp = ctypes.POINTER
    sig = {
        "culi_default_opts": (None, [pp(culi_opts)]),
        "culi_init": (I, [pp(culi_opts), pp(P)]),
        "culi_shutdown": (None, [P]),
        "culi_read": (I, [P, ctypes.c_char_p, SZ, pp(P), pp(SZ)]),
        "culi_image_nforms": (U32, [P]),
        "culi_image_nnodes": (U64, [P]),
        "culi_image_free": (None, [P]),
        "culi_define": (I, [P, P, pp(U32), pp(ctypes.c_uint8)]),
        "culi_eval_batch": (I, [P, P, pp(P)]),
        "culi_upload": (I, [P, P, pp(U32)]),
        "culi_eval_uploaded": (I, [P, U32]),
        "culi_fetch_results": (I, [P, U32, pp(P)]),
        "culi_release": (I, [P, U32]),
        "culi_results_count": (U32, [P]),
        "culi_result_info": (I, [P, U32, pp(ctypes.c_uint8), pp(ctypes.c_uint8), pp(U64)]),
        "culi_result_int": (I, [P, U32, pp(ctypes.c_int64)]),
        "culi_result_float": (I, [P, U32, pp(ctypes.c_double)]),
        "culi_print": (I, [P, U32, ctypes.c_char_p, SZ, pp(SZ)]),
        "culi_results_totals": (I, [P, pp(U64), pp(U32)]),
        "culi_results_free": (None, [P]),
        "culi_env_export": (I, [P, P, SZ, pp(SZ)]),
        "culi_env_import": (I, [P, P, SZ]),
        "culi_results_serialize": (I, [P, P, SZ, pp(SZ)]),
        "culi_results_merge": (I, [pp(P), pp(SZ), I, pp(pp(U32)), pp(P)]),
        "culi_status_string": (ctypes.c_char_p, [I]),
        "culi_error_name": (ctypes.c_char_p, [ctypes.c_uint8]),
        "culi_last_timing": (I, [P, pp(ctypes.c_float), pp(U32), pp(U64)]),
        "culi_records_device": (I, [P, P, SZ, pp(SZ)]),
        "culi_last_stats": (I, [P, pp(U32), pp(U32), pp(U32)]),
        "culi_last_splits": (I, [P, pp(U32)]),
        "culi_last_split_claims": (I, [P, pp(U32)]),
        "culi_last_waits": (I, [P, pp(U32), pp(U32)]),
        "culi_last_reruns": (I, [P, pp(U32), pp(U32)]),
        "culi_image_pin": (I, [P, pp(U64)]),
        "culi_results_wire_bytes": (I, [P, pp(U64)]),
        "culi_define_text": (I, [P, P, SZ, I, pp(U32), pp(ctypes.c_uint8), pp(SZ)]),
        "culi_eval_text": (I, [P, P, SZ, I, pp(P), pp(SZ)]),
        "culi_upload_text": (I, [P, P, SZ, I, pp(U32), pp(U32), pp(SZ)]),
        "culi_last_read": (I, [P, pp(ctypes.c_float), pp(U64), pp(U64)]),
        "culi_collect": (I, [P, pp(U64), pp(U64)]),
        "culi_heap_usage": (I, [P, pp(U64), pp(U64), pp(U64)]),
        "culi_arena_bytes": (I, [pp(culi_opts), pp(U64)]),
        "culi_eval_batch_async": (I, [P, P, pp(P)]),
        "culi_sync": (I, [P]),
        "culi_complete": (I, [P, U32]),
        "culi_results_export": (I, [P, P, SZ, pp(SZ)]),
        "culi_results_import": (I, [P, pp(P), pp(SZ), I, pp(pp(U32)), pp(P)]),
    }
    for name, (res, args) in sig.items():
        if os.environ.get("CULI_LIB") and not hasattr(L, name):   # an older A/B build: skip newer calls
            continue
        fn = getattr(L, name)
        fn.restype = res
        fn.argtypes = args
        globals()[name] = fn
    _lib = L
    return L


def _status_string(s: int) -> str:
    try:
        return load().culi_status_string(s).decode()
    except Exception:  # noqa: BLE001 - only for messages
        return "status"


def _check(rc: int, what: str) -> None:
    if rc != 0:
        raise CuliError(rc, what)


class ParseError(CuliError):
    def __init__(self, status: int, offset: int):
        self.offset = offset
        RuntimeError.__init__(self, "parse error at byte %d" % offset)
        self.status = status


class Image:
    def __init__(self, ptr: int):
        self._p = ctypes.c_void_p(ptr)

    @property
    def nforms(self) -> int:
        return load().culi_image_nforms(self._p)

    @property
    def nnodes(self) -> int:
        return load().culi_image_nnodes(self._p)

    def pin(self) -> int:
        """Page-lock the host arrays (uploads then DMA from pinned memory); returns the H2D bytes."""
        b = ctypes.c_uint64(0)
        _check(load().culi_image_pin(self._p, ctypes.byref(b)), "culi_image_pin")
        return b.value

    def __del__(self):
        if getattr(self, "_p", None) and self._p.value and _lib is not None:   # None at interpreter exit
            _lib.culi_image_free(self._p)
            self._p = None


class Results:
    def __init__(self, ptr: int):
        self._p = ctypes.c_void_p(ptr)

    def __len__(self) -> int:
        return load().culi_results_count(self._p)

    def info(self, i: int) -> tuple[int, int, int]:
        t, e, s = ctypes.c_uint8(), ctypes.c_uint8(), ctypes.c_uint64()
        _check(load().culi_result_info(self._p, i, ctypes.byref(t), ctypes.byref(e), ctypes.byref(s)),
               "culi_result_info")
        return t.value, e.value, s.value

    def print(self, i: int) -> str:
        L = load()
        need = ctypes.c_size_t(0)
        buf = ctypes.create_string_buffer(256)
        rc = L.culi_print(self._p, i, buf, 256, ctypes.byref(need))
        if rc != 0:
            buf = ctypes.create_string_buffer(need.value + 1)
            _check(L.culi_print(self._p, i, buf, need.value + 1, ctypes.byref(need)), "culi_print")
        return buf.value.decode()

    def printed(self) -> list[str]:
        return [self.print(i) for i in range(len(self))]

    def float_value(self, i: int) -> float:
        v = ctypes.c_double()
        _check(load().culi_result_float(self._p, i, ctypes.byref(v)), "culi_result_float")
        return v.value

    def int_value(self, i: int) -> int:
        v = ctypes.c_int64()
        _check(load().culi_result_int(self._p, i, ctypes.byref(v)), "culi_result_int")
        return v.value

    def steps(self) -> list[int]:
        return [self.info(i)[2] for i in range(len(self))]

    def errs(self) -> list[int]:
        return [self.info(i)[1] for i in range(len(self))]

    def totals(self) -> tuple[int, int]:
        s, e = ctypes.c_uint64(), ctypes.c_uint32()
        _check(load().culi_results_totals(self._p, ctypes.byref(s), ctypes.byref(e)), "culi_results_totals")
        return s.value, e.value

    def wire_bytes(self) -> int:
        """Bytes the fetch copied device -> host (records + value tokens)."""
        b = ctypes.c_uint64(0)
        _check(load().culi_results_wire_bytes(self._p, ctypes.byref(b)), "culi_results_wire_bytes")
        return b.value

    def serialize(self) -> bytes:
        L = load()
        need = ctypes.c_size_t(0)
        L.culi_results_serialize(self._p, None, 0, ctypes.byref(need))
        buf = ctypes.create_string_buffer(need.value)
        _check(L.culi_results_serialize(self._p, buf, need.value, ctypes.byref(need)),
               "culi_results_serialize")
        return buf.raw[: need.value]

    def __del__(self):
        if getattr(self, "_p", None) and self._p.value and _lib is not None:   # None at interpreter exit
            _lib.culi_results_free(self._p)
            self._p = None


def merge_results(blobs: list[bytes], form_index: list[list[int]]) -> Results:
    """culi_results_merge: rebuild one result set from per-rank serialized blobs."""
    L = load()
    n = len(blobs)
    bufs = [ctypes.create_string_buffer(b, len(b)) for b in blobs]
    ptrs = (ctypes.c_void_p * n)(*[ctypes.cast(b, ctypes.c_void_p) for b in bufs])
    sizes = (ctypes.c_size_t * n)(*[len(b) for b in blobs])
    idx_arrays = [(ctypes.c_uint32 * max(len(ix), 1))(*ix) for ix in form_index]
    idx_ptrs = (ctypes.POINTER(ctypes.c_uint32) * n)(
        *[ctypes.cast(a, ctypes.POINTER(ctypes.c_uint32)) for a in idx_arrays])
    out = ctypes.c_void_p()
    _check(L.culi_results_merge(ptrs, sizes, n, idx_ptrs, ctypes.byref(out)), "culi_results_merge")
    return Results(out.value)


class Context:
    """One CuLi session on one GPU (culi_init ... culi_shutdown)."""

    def __init__(self, device: int = 0, stream: int | None = None, heap_nodes: int = 0,
                 max_depth: int = 0, fuel: int = 0, vstack_entries: int = 0, slots: int = 0,
                 flags: int = 0, arena=None):
        """arena: optional caller-owned device memory (a CUDA uint8 tensor of at least
        Context.arena_bytes(...) bytes) for the heap, global frame, strings and stacks (culi_opts.heap_base)."""
        L = load()
        o = culi_opts()
        L.culi_default_opts(ctypes.byref(o))
        o.device = device
        o.stream = stream
        o.heap_nodes = heap_nodes
        o.max_depth = max_depth
        o.fuel = fuel
        o.vstack_entries = vstack_entries
        o.slots = slots
        o.flags = flags
        self._arena = arena                      # keep the caller's tensor alive as long as the ctx
        if arena is not None:
            o.heap_base = arena.data_ptr()
            o.heap_bytes = arena.numel() * arena.element_size()
        self.opts = o
        p = ctypes.c_void_p()
        _check(L.culi_init(ctypes.byref(o), ctypes.byref(p)), "culi_init")
        self._p = p

    def close(self) -> None:
        if getattr(self, "_p", None) and self._p.value:
            load().culi_shutdown(self._p)
            self._p = None

    def __del__(self):
        try:
            self.close()
        except Exception:  # noqa: BLE001 - interpreter shutdown (module globals already torn down)
            pass

    def read(self, text: str | bytes) -> Image:
        b = text.encode() if isinstance(text, str) else text
        out = ctypes.c_void_p()
        off = ctypes.c_size_t(0)
        rc = load().culi_read(self._p, b, len(b), ctypes.byref(out), ctypes.byref(off))
        if rc == -2:
            raise ParseError(rc, off.value)
        _check(rc, "culi_read")
        return Image(out.value)

    def define(self, defs: str | bytes | Image) -> None:
        img = defs if isinstance(defs, Image) else self.read(defs)
        fi = ctypes.c_uint32(0)
        fe = ctypes.c_uint8(0)
        rc = load().culi_define(self._p, img._p, ctypes.byref(fi), ctypes.byref(fe))
        if rc == -6:
            err = CuliError(rc, "culi_define (form %d: %s)" % (fi.value, ERR_NAMES[fe.value]))
            err.failed_index = fi.value
            err.failed_err = fe.value
            raise err
        _check(rc, "culi_define")

    # --- device reader: text -> heap on the GPU ----------------------------------------
    @staticmethod
    def _text(text):
        """(pointer, length, on_device, keepalive) for str / bytes (host) or a uint8 tensor (host or cuda)."""
        if isinstance(text, str):
            text = text.encode()
        if isinstance(text, (bytes, bytearray)):
            buf = ctypes.create_string_buffer(bytes(text), len(text))
            return ctypes.cast(buf, ctypes.c_void_p), len(text), 0, buf
        return ctypes.c_void_p(text.data_ptr()), text.numel() * text.element_size(), int(text.is_cuda), text

    def define_text(self, text) -> None:
        ptr, n, dev, keep = self._text(text)
        fi, fe, off = ctypes.c_uint32(0), ctypes.c_uint8(0), ctypes.c_size_t(0)
        rc = load().culi_define_text(self._p, ptr, n, dev, ctypes.byref(fi), ctypes.byref(fe), ctypes.byref(off))
        if rc == -2:
            raise ParseError(rc, off.value)
        if rc == -6:
            err = CuliError(rc, "culi_define_text (form %d: %s)" % (fi.value, ERR_NAMES[fe.value]))
            err.failed_index = fi.value
            err.failed_err = fe.value
            raise err
        _check(rc, "culi_define_text")

    def eval_text(self, text) -> Results:
        ptr, n, dev, keep = self._text(text)
        out, off = ctypes.c_void_p(), ctypes.c_size_t(0)
        rc = load().culi_eval_text(self._p, ptr, n, dev, ctypes.byref(out), ctypes.byref(off))
        if rc == -2:
            raise ParseError(rc, off.value)
        _check(rc, "culi_eval_text")
        return Results(out.value)

    def upload_text(self, text) -> tuple[int, int]:
        """Read on the device and prepare the batch; returns (handle, number of forms)."""
        ptr, n, dev, keep = self._text(text)
        h, nf, off = ctypes.c_uint32(0), ctypes.c_uint32(0), ctypes.c_size_t(0)
        rc = load().culi_upload_text(self._p, ptr, n, dev, ctypes.byref(h), ctypes.byref(nf), ctypes.byref(off))
        if rc == -2:
            raise ParseError(rc, off.value)
        _check(rc, "culi_upload_text")
        return h.value, nf.value

    def collect(self) -> tuple[int, int]:
        """culi_collect: compact the persistent heap segment now; (live nodes, freed nodes)."""
        a, b = ctypes.c_uint64(), ctypes.c_uint64()
        _check(load().culi_collect(self._p, ctypes.byref(a), ctypes.byref(b)), "culi_collect")
        return a.value, b.value

    def heap_usage(self) -> tuple[int, int, int]:
        """(persistent nodes in use, heap capacity, nodes reclaimed so far)."""
        a, b, c = ctypes.c_uint64(), ctypes.c_uint64(), ctypes.c_uint64()
        _check(load().culi_heap_usage(self._p, ctypes.byref(a), ctypes.byref(b), ctypes.byref(c)), "culi_heap_usage")
        return a.value, b.value, c.value

    def last_read(self) -> tuple[float, int, int]:
        """(device ms, items, nodes) of the last device read."""
        ms, it, nd = ctypes.c_float(), ctypes.c_uint64(), ctypes.c_uint64()
        _check(load().culi_last_read(self._p, ctypes.byref(ms), ctypes.byref(it), ctypes.byref(nd)),
               "culi_last_read")
        return ms.value, it.value, nd.value

    def eval_batch(self, forms: str | bytes | Image) -> Results:
        img = forms if isinstance(forms, Image) else self.read(forms)
        out = ctypes.c_void_p()
        _check(load().culi_eval_batch(self._p, img._p, ctypes.byref(out)), "culi_eval_batch")
        return Results(out.value)

    def upload(self, forms: str | bytes | Image) -> int:
        img = forms if isinstance(forms, Image) else self.read(forms)
        self._uploaded_image = img
        h = ctypes.c_uint32(0)
        _check(load().culi_upload(self._p, img._p, ctypes.byref(h)), "culi_upload")
        return h.value

    def eval_uploaded(self, handle: int) -> None:
        _check(load().culi_eval_uploaded(self._p, handle), "culi_eval_uploaded")

    def fetch_results(self, handle: int) -> Results:
        out = ctypes.c_void_p()
        _check(load().culi_fetch_results(self._p, handle, ctypes.byref(out)), "culi_fetch_results")
        return Results(out.value)

    def release(self, handle: int) -> None:
        _check(load().culi_release(self._p, handle), "culi_release")

    def last_timing(self) -> tuple[list[float], int, int]:
        ms = (ctypes.c_float * 3)()
        k = ctypes.c_uint32()
        h = ctypes.c_uint64()
        _check(load().culi_last_timing(self._p, ms, ctypes.byref(k), ctypes.byref(h)), "culi_last_timing")
        return list(ms), k.value, h.value

    def last_stats(self) -> tuple[int, int]:
        """(forms handled by the fan-out kernels, forms re-evaluated sequentially) of the last batch."""
        a, b, c = ctypes.c_uint32(), ctypes.c_uint32(), ctypes.c_uint32()
        _check(load().culi_last_stats(self._p, ctypes.byref(a), ctypes.byref(b), ctypes.byref(c)),
               "culi_last_stats")
        self.last_nested = c.value
        return a.value, b.value

    def last_splits(self) -> int:
        """Split groups published by the last batch (argument splitting)."""
        g = ctypes.c_uint32()
        _check(load().culi_last_splits(self._p, ctypes.byref(g)), "culi_last_splits")
        return g.value

    def last_split_claims(self) -> int:
        """Split tasks of the last batch that an idle lane claimed (the rest were taken back)."""
        g = ctypes.c_uint32()
        _check(load().culi_last_split_claims(self._p, ctypes.byref(g)), "culi_last_split_claims")
        return g.value

    def last_waits(self) -> tuple[int, list[int]]:
        """Bounded inter-warp waits that gave up in the last fetched batch (0 in a healthy run) and the first
        one's state: [kind (1 join, 2 queue, 3 nested), group, lane, form, state, mask, remaining, done,
        claimer]."""
        n = ctypes.c_uint32()
        d = (ctypes.c_uint32 * 9)()
        _check(load().culi_last_waits(self._p, ctypes.byref(n), d), "culi_last_waits")
        return n.value, list(d)

    @staticmethod
    def arena_bytes(device: int = 0, heap_nodes: int = 0, max_depth: int = 0, vstack_entries: int = 0,
                    slots: int = 0) -> int:
        """Bytes a caller-owned arena needs for these sizes (culi_arena_bytes)."""
        o = culi_opts()
        load().culi_default_opts(ctypes.byref(o))
        o.device, o.heap_nodes, o.max_depth, o.vstack_entries, o.slots = device, heap_nodes, max_depth, \
            vstack_entries, slots
        b = ctypes.c_uint64(0)
        _check(load().culi_arena_bytes(ctypes.byref(o), ctypes.byref(b)), "culi_arena_bytes")
        return b.value

    def eval_batch_async(self, forms: str | bytes | Image) -> "Results":
        """Start a batch (culi_eval_batch_async); the results are ready after sync()."""
        img = forms if isinstance(forms, Image) else self.read(forms)
        out = ctypes.c_void_p()
        _check(load().culi_eval_batch_async(self._p, img._p, ctypes.byref(out)), "culi_eval_batch_async")
        r = Results(out.value)
        r._image = img                           # the image must live until culi_sync
        return r

    def sync(self) -> None:
        _check(load().culi_sync(self._p), "culi_sync")

    def complete(self, handle: int) -> None:
        """Finish the uploaded batch's device-resident results (fallbacks, payload regrowth), no D2H."""
        _check(load().culi_complete(self._p, handle), "culi_complete")

    def results_export_size(self) -> int:
        need = ctypes.c_size_t(0)
        _check(load().culi_results_export(self._p, None, 0, ctypes.byref(need)), "culi_results_export")
        return need.value

    def results_export(self, dev_ptr: int, cap: int) -> int:
        """Pack the current batch's device-resident results into dev_ptr[cap] (stream-ordered, no sync)."""
        used = ctypes.c_size_t(0)
        _check(load().culi_results_export(self._p, ctypes.c_void_p(dev_ptr), cap, ctypes.byref(used)),
               "culi_results_export")
        return used.value

    def results_import(self, dev_ptrs: list[int], sizes: list[int],
                       form_index: list[list[int]] | None = None) -> "Results":
        """Merge per-rank exported device buffers into one host result set (None: strided deal)."""
        n = len(dev_ptrs)
        ptrs = (ctypes.c_void_p * n)(*dev_ptrs)
        szs = (ctypes.c_size_t * n)(*sizes)
        idx = None
        keep = []
        if form_index is not None:
            arrs = [(ctypes.c_uint32 * len(ix))(*ix) for ix in form_index]
            keep = arrs
            idx = (ctypes.POINTER(ctypes.c_uint32) * n)(*[ctypes.cast(a, ctypes.POINTER(ctypes.c_uint32))
                                                         for a in arrs])
        out = ctypes.c_void_p()
        _check(load().culi_results_import(self._p, ptrs, szs, n, idx, ctypes.byref(out)), "culi_results_import")
        del keep
        return Results(out.value)

    def last_reruns(self) -> tuple[int, int]:
        """(forms re-evaluated by the sequential fallback, payload-buffer regrowths) of the last fetch."""
        a, b = ctypes.c_uint32(), ctypes.c_uint32()
        _check(load().culi_last_reruns(self._p, ctypes.byref(a), ctypes.byref(b)), "culi_last_reruns")
        return a.value, b.value

    def records_device(self, dev_ptr: int | None, cap: int = 0) -> int:
        need = ctypes.c_size_t(0)
        _check(load().culi_records_device(self._p, ctypes.c_void_p(dev_ptr) if dev_ptr else None, cap,
                                          ctypes.byref(need)), "culi_records_device")
        return need.value

    # --- distributed hooks -------------------------------------------------------------------------
    def env_export_size(self) -> int:
        need = ctypes.c_size_t(0)
        load().culi_env_export(self._p, None, 0, ctypes.byref(need))
        return need.value

    def env_export(self, dev_ptr: int, cap: int) -> int:
        need = ctypes.c_size_t(0)
        _check(load().culi_env_export(self._p, ctypes.c_void_p(dev_ptr), cap, ctypes.byref(need)),
               "culi_env_export")
        return need.value

    def env_import(self, dev_ptr: int, nbytes: int) -> None:
        _check(load().culi_env_import(self._p, ctypes.c_void_p(dev_ptr), nbytes), "culi_env_import")
