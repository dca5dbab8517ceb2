"""Build liblns.so in-tree with nvcc for sm_100a (B200)."""
from __future__ import annotations

import os
import subprocess
import sys

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
SRC = [os.path.join(PKG, "csrc", "lns.cu")]
DEPS = [os.path.join(PKG, "csrc", "bqp.cuh")]  # included by lns.cu
HDR = [os.path.join(ROOT, "include", "lns.h")]
LIB = os.path.join(PKG, "liblns.so")

NVCC_FLAGS = [
    "-gencode", "arch=compute_100a,code=sm_100a",
    "-O3", "-lineinfo", "-std=c++17",
    "-Xcompiler", "-fPIC,-O2", "-shared",
]


def source_hash() -> str:
    """sha256 (16 hex) of everything that determines the kernels' SASS: the CUDA sources, the header
    and the nvcc flags. A committed ncu capture records it; bench.py refuses a capture whose hash
    differs from the current sources (its per-neighbour instruction counts would be stale)."""
    import hashlib

    h = hashlib.sha256()
    for p in SRC + DEPS + HDR:
        with open(p, "rb") as fh:
            h.update(fh.read())
    h.update(" ".join(NVCC_FLAGS).encode())
    return h.hexdigest()[:16]


def nvcc() -> str:
    for cand in (os.environ.get("NVCC"), "/usr/local/cuda/bin/nvcc", "nvcc"):
        if cand and (os.path.sep not in cand or os.path.exists(cand)):
            return cand
    return "nvcc"


def stale() -> bool:
    if not os.path.exists(LIB):
        return True
    t = os.path.getmtime(LIB)
    return any(os.path.getmtime(p) > t for p in SRC + DEPS + HDR)


LIB_PROF = os.path.join(PKG, "liblns_prof.so")  # -DLNS_PHASE_TIMING variant for tools/profiling


def build(force: bool = False, verbose: bool = False, profiling: bool = False) -> str:
    lib = LIB_PROF if profiling else LIB
    if not force and not profiling and not stale():
        return LIB
    tmp = lib + f".tmp{os.getpid()}"
    extra = ["-DLNS_PHASE_TIMING"] if profiling else []
    cmd = [nvcc(), *NVCC_FLAGS, *extra, "-I", os.path.join(ROOT, "include"), "-o", tmp, *SRC, "-ldl"]
    if verbose:
        cmd.insert(1, "-Xptxas=-v")
        print(" ".join(cmd), file=sys.stderr)
    subprocess.check_call(cmd)
    os.replace(tmp, lib)
    return lib


def build_variant(name: str, defines: list[str]) -> str:
    """Experimental build with extra -D flags into build/variants/liblns_<name>.so (LNS_LIB=... selects it)."""
    out_dir = os.path.join(ROOT, "build", "variants")
    os.makedirs(out_dir, exist_ok=True)
    lib = os.path.join(out_dir, f"liblns_{name}.so")
    cmd = [nvcc(), *NVCC_FLAGS, *[f"-D{d}" for d in defines], "-I", os.path.join(ROOT, "include"), "-o", lib, *SRC, "-ldl"]
    subprocess.check_call(cmd)
    return lib


if __name__ == "__main__":
    print(build(force="--force" in sys.argv, verbose="-v" in sys.argv, profiling="--profiling" in sys.argv))
