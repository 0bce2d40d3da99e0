"""Build libculi.so in-tree with nvcc for sm_100a (no JIT, no torch extension machinery needed)."""
from __future__ import annotations

import os
import subprocess
import sys

HERE = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(HERE)
CSRC = os.path.join(HERE, "csrc")
LIB = os.path.join(HERE, "libculi.so")
SOURCES = ["culi_host.cpp", "culi_kernels.cu", "culi_dispatch.cu", "culi_capi.cu", "culi_dist.cu", "culi_reader.cu", "culi_gc.cu"]
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]
FLAGS = ["-O3", "-std=c++17", "-lineinfo", "--fmad=false", "-Xcompiler", "-fPIC,-O2,-ffp-contract=off",
         "-I" + os.path.join(ROOT, "include"), "-I" + CSRC]


def _stale(target: str, deps: list[str]) -> bool:
    if not os.path.exists(target):
        return True
    t = os.path.getmtime(target)
    return any(os.path.getmtime(d) > t for d in deps)


def build(verbose: bool = False, force: bool = False, ptxas_v: bool = False, defines: list[str] | None = None,
          out: str | None = None) -> str:
    """defines / out: debug or A/B variants (e.g. ["CULI_WATCHDOG=20000"], "scratch/libculi_wd.so")."""
    if defines or out:
        return _build_variant(defines or [], out or LIB, verbose)
    if HERE not in sys.path:
        sys.path.insert(0, HERE)
    import gen_pow5
    gen_pow5.write(os.path.join(CSRC, "culi_pow5.inc"))
    deps = [os.path.join(CSRC, f) for f in os.listdir(CSRC)] + [os.path.join(ROOT, "include", "culi.h")]
    if not force and not _stale(LIB, deps):
        return LIB
    objs, cmds = [], []
    for src in SOURCES:
        obj = os.path.join(CSRC, src + ".o")
        cmd = [NVCC, *ARCH, *FLAGS, "-c", os.path.join(CSRC, src), "-o", obj]
        if ptxas_v and src.endswith(".cu"):
            cmd += ["-Xptxas", "-v"]
        if verbose:
            print(" ".join(cmd), file=sys.stderr)
        cmds.append(cmd)
        objs.append(obj)
    _compile_all(cmds)
    cmd = [NVCC, *ARCH, "-shared", "-o", LIB, *objs, "-lcudart"]
    subprocess.check_call(cmd)
    for o in objs:
        os.remove(o)
    return LIB


def _compile_all(cmds: list[list[str]]) -> None:
    """Translation units compile in parallel (one nvcc per unit); any failure raises."""
    from concurrent.futures import ThreadPoolExecutor
    with ThreadPoolExecutor(max_workers=max(1, min(len(cmds), os.cpu_count() or 1))) as ex:
        for f in [ex.submit(subprocess.check_call, c) for c in cmds]:
            f.result()


def _build_variant(defines: list[str], out: str, verbose: bool) -> str:
    import tempfile
    tmp = tempfile.mkdtemp()
    objs, cmds = [], []
    for src in SOURCES:
        obj = os.path.join(tmp, src + ".o")
        cmd = [NVCC, *ARCH, *FLAGS, *["-D" + d for d in defines], "-c", os.path.join(CSRC, src), "-o", obj]
        if verbose:
            print(" ".join(cmd), file=sys.stderr)
        cmds.append(cmd)
        objs.append(obj)
    _compile_all(cmds)
    subprocess.check_call([NVCC, *ARCH, "-shared", "-o", out, *objs, "-lcudart"])
    return out


if __name__ == "__main__":
    build(verbose=True, force=True, ptxas_v="-v" in sys.argv)
