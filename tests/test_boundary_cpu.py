"""CPU tests of the C-ABI boundary: libculi.so builds for sm_100a, loads, exports every entry point
include/culi.h declares, fails loudly without a GPU, and its host-only result merge/print logic works."""
from __future__ import annotations

import ctypes
import os
import re
import struct

import pytest

from tests import wire

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def lib():
    from paper_conf_cluster_subdbn18_b200 import build, culi
    build.build()
    return culi, culi.load()


def header_symbols():
    text = open(os.path.join(ROOT, "include", "culi.h")).read()
    text = re.sub(r"/\*.*?\*/", "", text, flags=re.S)
    return sorted(set(re.findall(r"\b(culi_[a-z_]+)\s*\(", text)))


def test_exports_every_declared_symbol(lib):
    culi, L = lib
    names = header_symbols()
    assert len(names) >= 25
    for n in names:
        assert hasattr(L, n), n
    assert sorted(culi.SYMBOLS) == names


def test_sm100a_cubin_present():
    from paper_conf_cluster_subdbn18_b200 import build
    import subprocess
    out = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "--list-elf", build.LIB], capture_output=True,
                         text=True).stdout
    assert "sm_100a" in out


def test_status_strings(lib):
    culi, L = lib
    assert L.culi_status_string(0) == b"ok"
    assert L.culi_status_string(-4) == b"CUDA error"
    assert L.culi_error_name(4) == b"SYNTAX"


def test_init_fails_loudly_without_gpu(lib):
    import torch
    if torch.cuda.is_available():
        pytest.skip("a GPU is present")
    culi, L = lib
    with pytest.raises(culi.CuliError) as ei:
        culi.Context()
    assert ei.value.status == -4


def test_merge_reorders_and_reinterns(lib):
    culi, _ = lib
    # rank 0 holds forms 0, 2; rank 1 holds forms 1, 3 (strided shards)
    r0 = wire.blob([(wire.INT, 0, 4, 7), (wire.SYM, 0, 1, wire.sym_id("foo", ["foo"]))], names=["foo"])
    # rank 1 interned "bar" before "foo", so its ids differ; one list result (1 bar) and one error
    extra1 = ["bar", "foo"]
    r1 = wire.blob([(wire.CONS, 0, 5, 0 | (4 << 32)), (13, 3, 4, 0)],
                   payload=[(wire.CONS, 0), (wire.INT, 1), (wire.CONS, 0), (wire.SYM, wire.sym_id("bar", extra1)),
                            (wire.NIL, 0)],
                   names=extra1)
    m = culi.merge_results([r0, r1], [[0, 2], [1, 3]])
    assert m.printed() == ["7", "(1 bar)", "foo", "#<error DIV0>"]
    assert m.steps() == [4, 5, 1, 4]


def test_merge_strings_and_floats(lib):
    culi, _ = lib
    f = struct.unpack("<Q", struct.pack("<d", -0.0))[0]
    r0 = wire.blob([(wire.STR, 0, 1, 0 | (1 << 32)), (wire.FLOAT, 0, 3, f)], payload=[(wire.STR, 0 | (2 << 32))],
                   strings=b"hi")
    r1 = wire.blob([(wire.STR, 0, 1, 0 | (1 << 32))], payload=[(wire.STR, 0 | (3 << 32))], strings=b"abc")
    m = culi.merge_results([r0, r1], [[0, 2], [1]])
    assert m.printed() == ['"hi"', '"abc"', "-0.0"]


def test_merge_rejects_bad_indices(lib):
    culi, _ = lib
    r0 = wire.blob([(wire.INT, 0, 1, 1)])
    with pytest.raises(culi.CuliError):
        culi.merge_results([r0, r0], [[0], [0]])          # duplicate form index
    with pytest.raises(culi.CuliError):
        culi.merge_results([b"junk" * 20], [[0]])


def test_serialize_roundtrip(lib):
    culi, _ = lib
    r = culi.merge_results([wire.blob([(wire.INT, 0, 9, 42)])], [[0]])
    again = culi.merge_results([r.serialize()], [[0]])
    assert again.printed() == ["42"] and again.steps() == [9]
