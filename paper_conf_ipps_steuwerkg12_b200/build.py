"""Builds the in-tree CUDA library ``liblmosem.so`` for sm_100a with nvcc.

The library is built in-tree (not into site-packages or a JIT cache) so that it travels
to the GPU box with the repo snapshot and is visibly the code the tests and bench load.
"""
from __future__ import annotations

import glob
import os
import subprocess
import sys

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
SO = os.path.join(PKG, "liblmosem.so")
L2PEAK_SO = os.path.join(PKG, "libl2peak.so")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]


def nccl_paths():
    """Include/lib dirs of the NCCL that torch loads (the venv's nvidia-nccl wheel)."""
    for base in sys.path:
        d = os.path.join(base, "nvidia", "nccl")
        if os.path.exists(os.path.join(d, "include", "nccl.h")):
            return os.path.join(d, "include"), os.path.join(d, "lib")
    return "/usr/include", "/usr/lib/x86_64-linux-gnu"


def _sources():
    return sorted(glob.glob(os.path.join(CSRC, "*.cu")) + glob.glob(os.path.join(CSRC, "*.cuh"))
                  + [os.path.join(ROOT, "include", "lmosem.h")])


def needs_build() -> bool:
    if not os.path.exists(SO) or not os.path.exists(L2PEAK_SO):
        return True
    t = min(os.path.getmtime(SO), os.path.getmtime(L2PEAK_SO))
    return any(os.path.getmtime(s) > t for s in _sources() + [os.path.join(ROOT, "include", "l2peak.h")])


def build_l2peak() -> str:
    tmp = L2PEAK_SO + f".tmp{os.getpid()}"
    cmd = [NVCC, *ARCH, "-O3", "-std=c++17", "-lineinfo", "-Xcompiler", "-fPIC,-fvisibility=hidden", "-shared",
           "-I", os.path.join(ROOT, "include"), os.path.join(CSRC, "l2peak.cu"), "-o", tmp]
    res = subprocess.run(cmd, capture_output=True, text=True)
    if res.returncode != 0:
        raise RuntimeError("nvcc failed:\n" + res.stdout + res.stderr)
    os.replace(tmp, L2PEAK_SO)
    return L2PEAK_SO


def build(force: bool = False, verbose: bool = False, defines=(), out: str | None = None,
          csrc: str | None = None, extra=()) -> str:
    """Builds liblmosem.so (and libl2peak.so). `defines`/`out` build an A/B variant of
    the kernels (e.g. defines=["LMK_TRASH=0"], out=".../liblmosem_v.so"); `csrc` compiles
    a modified copy of the sources (tools/gpu_mutants.py) into `out`; `extra` adds nvcc flags."""
    src_dir = csrc or CSRC
    if out is None and not force and not needs_build():
        return SO
    target = out or SO
    if out is None:
        build_l2peak()
    inc, lib = nccl_paths()
    tmp = target + f".tmp{os.getpid()}"
    cmd = [NVCC, *ARCH, "-O3", "-std=c++17", "-lineinfo", "-Xptxas", "-v", *[f"-D{d}" for d in defines], *extra,
           "-Xcompiler", "-fPIC,-fvisibility=hidden", "-shared",
           "-I", os.path.join(ROOT, "include"), "-I", src_dir, "-I", inc,
           os.path.join(src_dir, "lmosem.cu"), "-o", tmp,
           "-L", lib, "-l:libnccl.so.2", f"-Xlinker=-rpath={lib}", "-lpthread"]
    res = subprocess.run(cmd, capture_output=True, text=True)
    if res.returncode != 0:
        raise RuntimeError("nvcc failed:\n" + res.stdout + res.stderr)
    if out is None:
        with open(os.path.join(PKG, "build_ptxas.log"), "w") as fh:
            fh.write(" ".join(cmd) + "\n" + res.stdout + res.stderr)
    if verbose:
        print(res.stderr)
    os.replace(tmp, target)
    return target


if __name__ == "__main__":
    print(build(force="--force" in sys.argv, verbose=True))
