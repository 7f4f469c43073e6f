"""Build the in-tree CUDA library ``lib/librs_lowrank.so`` for sm_100a with nvcc.

Each ``csrc/*.cu`` is compiled separately (``-gencode arch=compute_100a,code=sm_100a -lineinfo``)
and linked into one shared library exporting the C ABI of ``include/rs_lowrank.h``.  NCCL comes
from the torch-bundled wheel (``nvidia/nccl``) so the process loads a single libnccl.
"""

from __future__ import annotations

import hashlib
import os
import subprocess
import sys
from concurrent.futures import ThreadPoolExecutor

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
LIBDIR = os.path.join(PKG, "lib")
LIB = os.path.join(LIBDIR, "librs_lowrank.so")
STAMP = os.path.join(LIBDIR, ".build_hash")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]


def _nccl_dirs():
    import importlib.util

    spec = importlib.util.find_spec("nvidia.nccl")
    cands = []
    if spec and spec.submodule_search_locations:
        cands += list(spec.submodule_search_locations)
    cands.append("/usr")
    for c in cands:
        inc = os.path.join(c, "include")
        lib = os.path.join(c, "lib")
        if os.path.exists(os.path.join(inc, "nccl.h")):
            if os.path.exists(os.path.join(lib, "libnccl.so.2")):
                return inc, lib
            lib = os.path.join(c, "lib", "x86_64-linux-gnu")
            if os.path.exists(os.path.join(lib, "libnccl.so.2")):
                return inc, lib
    raise RuntimeError("nccl.h / libnccl.so.2 not found")


def _sources():
    return sorted(os.path.join(CSRC, f) for f in os.listdir(CSRC) if f.endswith(".cu"))


def _hash(files):
    h = hashlib.sha256()
    for f in sorted(files):
        with open(f, "rb") as fh:
            h.update(os.path.relpath(f, ROOT).encode())  # location-independent (the repo is copied to the GPU box)
            h.update(fh.read())
    return h.hexdigest()


def build(force: bool = False, verbose: bool = False) -> str:
    srcs = _sources()
    deps = srcs + [os.path.join(CSRC, f) for f in os.listdir(CSRC) if f.endswith((".cuh", ".h"))]
    deps.append(os.path.join(ROOT, "include", "rs_lowrank.h"))
    deps.append(os.path.abspath(__file__))
    extra = os.environ.get("RS_EXTRA_NVCC_FLAGS", "").split()  # development experiments only
    digest = _hash(deps) + ("|" + " ".join(extra) if extra else "")
    # the stamp (git-ignored) records the source digest AND the digest of the .so it was written
    # with, so a .so replaced by another revision's (a sync, a checkout) is never taken as current
    if not force and os.path.exists(LIB) and os.path.exists(STAMP):
        with open(STAMP) as fh:
            if fh.read().strip() == digest + ":" + _hash([LIB]):
                return LIB
    os.makedirs(LIBDIR, exist_ok=True)
    nccl_inc, nccl_lib = _nccl_dirs()
    common = ["nvcc", *ARCH, "-O3", "-lineinfo", "-std=c++17", "-Xcompiler", "-fPIC", "-Xcompiler", "-fvisibility=hidden",
              f"-I{os.path.join(ROOT, 'include')}", f"-I{CSRC}", f"-I{nccl_inc}", *extra]
    objs = []

    def compile_one(src):
        obj = os.path.join(LIBDIR, os.path.basename(src)[:-3] + ".o")
        cmd = common + ["-c", src, "-o", obj]
        if verbose:
            print(" ".join(cmd), file=sys.stderr)
        r = subprocess.run(cmd, capture_output=True, text=True)
        if r.returncode != 0:
            raise RuntimeError(f"nvcc failed for {src}:\n{r.stdout}\n{r.stderr}")
        return obj

    with ThreadPoolExecutor(max_workers=min(8, os.cpu_count() or 1)) as ex:
        objs = list(ex.map(compile_one, srcs))
    link = ["nvcc", *ARCH, "-shared", "-Xcompiler", "-fPIC", "-o", LIB + ".tmp", *objs,
            f"-L{nccl_lib}", "-l:libnccl.so.2", f"-Xlinker", f"-rpath={nccl_lib}", "-lcuda" if False else "-lcudart_static"]
    r = subprocess.run(link, capture_output=True, text=True)
    if r.returncode != 0:
        raise RuntimeError(f"link failed:\n{r.stdout}\n{r.stderr}")
    os.replace(LIB + ".tmp", LIB)
    for o in objs:
        os.remove(o)
    with open(STAMP, "w") as fh:
        fh.write(digest + ":" + _hash([LIB]))
    return LIB


if __name__ == "__main__":
    print(build(force="--force" in sys.argv, verbose="-v" in sys.argv))
