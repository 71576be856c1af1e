"""Build the CUDA C-ABI library (sm_100a) in-tree with nvcc.

The product is ``paper_conf_cluster_mcintosh_smithm17_b200/libtea_b200.so``:
hand-written CUDA kernels + the host driver behind ``include/tea.h``. It links
NCCL from the Python environment (the same libnccl.so.2 that torch loads) and
the static CUDA runtime.
"""
from __future__ import annotations

import glob
import os
import subprocess
import sys

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
INCLUDE = os.path.join(ROOT, "include")
LIB = os.path.join(PKG, "libtea_b200.so")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]


def nccl_dir() -> str:
    for p in sys.path:
        d = os.path.join(p, "nvidia", "nccl")
        if os.path.exists(os.path.join(d, "include", "nccl.h")):
            return d
    raise RuntimeError("NCCL headers (nvidia/nccl) not found in the Python environment")


def sources():
    return sorted(glob.glob(os.path.join(CSRC, "*.cu")))


def deps():
    return sources() + sorted(glob.glob(os.path.join(CSRC, "*.h"))) + [
        os.path.join(INCLUDE, "tea.h")]


def stale() -> bool:
    if not os.path.exists(LIB):
        return True
    t = os.path.getmtime(LIB)
    return any(os.path.getmtime(f) > t for f in deps())


def nvtx_include() -> str:
    for p in sys.path:
        d = os.path.join(p, "nvidia", "nvtx", "include")
        if os.path.exists(os.path.join(d, "nvtx3", "nvToolsExt.h")):
            return d
    return "/usr/local/cuda/include"  # the toolkit ships nvtx3 too


def nvcc_cmd(out: str, extra=()):
    nccl = nccl_dir()
    return ["nvcc", "-O3", "-std=c++17", *ARCH, "-lineinfo", "-Xcompiler", "-fPIC", "-shared",
            "-I" + INCLUDE, "-I" + os.path.join(nccl, "include"), "-I" + nvtx_include(),
            "-L" + os.path.join(nccl, "lib"), "-l:libnccl.so.2",
            "-Xlinker", "-rpath," + os.path.join(nccl, "lib"),
            *extra, "-o", out, *sources()]


def build(force: bool = False, verbose: bool = False) -> str:
    if not force and not stale():
        return LIB
    tmp = LIB + f".tmp{os.getpid()}"
    cmd = nvcc_cmd(tmp)
    if verbose:
        print(" ".join(cmd))
    subprocess.check_call(cmd)
    os.replace(tmp, LIB)
    return LIB


if __name__ == "__main__":
    print(build(force="--force" in sys.argv, verbose=True))
