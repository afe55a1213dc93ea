"""Build the in-tree CUDA library libmpcgs.so for sm_100a with nvcc.

The library is a plain shared object with a C ABI (include/mpcgs.h); it links
the CUDA runtime statically and loads NCCL with dlopen only when world > 1.
"""
from __future__ import annotations

import concurrent.futures
import glob
import os
import shutil
import subprocess
import sys

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
INCLUDE = os.path.join(ROOT, "include")
LIB = os.path.join(PKG, "libmpcgs.so")

NVCC_FLAGS = [
    "-std=c++17", "-O3", "-lineinfo", "-Xcompiler", "-fPIC",
    "-gencode", "arch=compute_100a,code=sm_100a",
    "--expt-relaxed-constexpr", "-Xptxas", "-v",
]


def sources():
    return sorted(glob.glob(os.path.join(CSRC, "*.cu")))


def headers():
    return sorted(glob.glob(os.path.join(CSRC, "*.cuh"))) + [os.path.join(INCLUDE, "mpcgs.h")]


def stale() -> bool:
    if not os.path.exists(LIB):
        return True
    t = os.path.getmtime(LIB)
    return any(os.path.getmtime(p) > t for p in sources() + headers())


def build(force: bool = False, verbose: bool = False, out: str = LIB, defines=()) -> str:
    """Compile libmpcgs.so (or a tuning variant with extra -D defines at `out`)."""
    if not force and out == LIB and not stale():
        return LIB
    nvcc = os.environ.get("NVCC", "nvcc")
    tmp = out + f".tmp{os.getpid()}"
    objdir = tmp + ".o.d"
    os.makedirs(objdir, exist_ok=True)
    srcs = sources()
    objs = [os.path.join(objdir, os.path.basename(src) + ".o") for src in srcs]
    base = [nvcc, *NVCC_FLAGS, *[f"-D{d}" for d in defines], "-I", INCLUDE, "-I", CSRC]

    def compile_one(src_obj):  # one translation unit per nvcc process, all in parallel
        src, obj = src_obj
        return subprocess.run([*base, "-c", "-o", obj, src], capture_output=True, text=True)

    with concurrent.futures.ThreadPoolExecutor(max_workers=max(1, min(len(srcs), os.cpu_count() or 1))) as ex:
        results = list(ex.map(compile_one, zip(srcs, objs)))
    log = "".join(r.stdout + r.stderr for r in results)
    if any(r.returncode != 0 for r in results):
        sys.stderr.write(log)
        shutil.rmtree(objdir, ignore_errors=True)
        raise RuntimeError("nvcc failed building libmpcgs.so")
    # the link carries the arch too: without it nvcc adds an (empty) sm_52 device-link image
    res = subprocess.run([nvcc, "-shared", "-gencode", "arch=compute_100a,code=sm_100a", "-Xcompiler", "-fPIC",
                          "-o", tmp, *objs, "-ldl"], capture_output=True,
                         text=True)
    shutil.rmtree(objdir, ignore_errors=True)
    if res.returncode != 0:
        sys.stderr.write(res.stdout + res.stderr)
        raise RuntimeError("nvcc failed linking libmpcgs.so")
    res.stderr = log
    if verbose:
        sys.stderr.write(log)
    if out == LIB:
        with open(os.path.join(PKG, "build_ptxas.log"), "w") as f:
            f.write(res.stderr)
    os.replace(tmp, out)
    return out


if __name__ == "__main__":
    build(force="--force" in sys.argv, verbose=True)
    print(LIB)
