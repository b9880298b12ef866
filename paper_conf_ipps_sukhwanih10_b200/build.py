"""Build libdock.so in-tree with nvcc for sm_100a (no JIT, no torch extension cache)."""
from __future__ import annotations

import glob
import os
import subprocess
import sys

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
LIB = os.path.join(PKG, "libdock.so")
# dock.cu = host logic + small kernels; launch_*.cu = one correlation-kernel family each (compiled in
# parallel, then linked into one shared library)
SOURCES = [os.path.join(CSRC, "dock.cu")] + sorted(glob.glob(os.path.join(CSRC, "launch_*.cu"))) + \
    [os.path.join(CSRC, "fft_engine.cu"), os.path.join(CSRC, "em.cu")]
HEADERS = (sorted(glob.glob(os.path.join(CSRC, "*.cuh"))) + sorted(glob.glob(os.path.join(CSRC, "*.h"))) +
           sorted(glob.glob(os.path.join(ROOT, "include", "*.h"))))

NVCC_FLAGS = [
    "-gencode", "arch=compute_100a,code=sm_100a",
    "-O3", "-lineinfo", "-std=c++17",
    "-Xcompiler", "-fPIC",
    "-Xptxas", "-v",
]


def _nvcc() -> str:
    for c in (os.environ.get("NVCC"), "/usr/local/cuda/bin/nvcc", "nvcc"):
        if c and (os.path.isabs(c) and os.path.exists(c) or not os.path.isabs(c)):
            return c
    return "nvcc"


STAMP = os.path.join(PKG, "libdock.defs")   # the DOCK_NVCC_DEFS the library was built with


def _defs() -> str:
    return " ".join(os.environ.get("DOCK_NVCC_DEFS", "").split())


def stale() -> bool:
    """Rebuild when a source is newer than the library, or when the experiment defines (DOCK_NVCC_DEFS)
    differ from those the library was built with (a tuning build is never silently reused)."""
    if not os.path.exists(LIB):
        return True
    try:
        with open(STAMP) as f:
            if f.read().strip() != _defs():
                return True
    except OSError:
        return True
    t = os.path.getmtime(LIB)
    return any(os.path.getmtime(p) > t for p in SOURCES + HEADERS)


def build_native(force: bool = False, verbose: bool = False) -> str:
    if not force and not stale():
        return LIB
    from concurrent.futures import ThreadPoolExecutor
    tag = f".tmp{os.getpid()}"
    objs = [os.path.join(PKG, "build", os.path.basename(s) + tag + ".o") for s in SOURCES]
    os.makedirs(os.path.join(PKG, "build"), exist_ok=True)

    def compile_one(src_obj):
        src, obj = src_obj
        # DOCK_NVCC_DEFS: extra -D flags for tuning experiments (e.g. "-DDOCK_TC_STAIR=2"); unset in normal builds
        extra = os.environ.get("DOCK_NVCC_DEFS", "").split()
        cmd = [_nvcc(), *NVCC_FLAGS, *extra, "-I", os.path.join(ROOT, "include"), "-c", "-o", obj, src]
        return subprocess.run(cmd, capture_output=True, text=True)

    with ThreadPoolExecutor(max_workers=max(1, min(len(SOURCES), os.cpu_count() or 1))) as ex:
        results = list(ex.map(compile_one, zip(SOURCES, objs)))
    log = ""
    for src, res in zip(SOURCES, results):
        log += f"== {os.path.basename(src)}\n" + res.stderr
        if res.returncode != 0:
            sys.stderr.write(res.stdout + res.stderr)
            raise RuntimeError(f"nvcc failed compiling {os.path.basename(src)}")
    tmp = LIB + tag
    res = subprocess.run([_nvcc(), "-gencode", "arch=compute_100a,code=sm_100a", "-shared", "-o", tmp, *objs,
                          "-lcuda", "-lcufft"], capture_output=True, text=True)
    if res.returncode != 0:
        sys.stderr.write(res.stdout + res.stderr)
        raise RuntimeError("nvcc failed linking libdock.so")
    for o in objs:
        os.remove(o)
    if verbose:
        sys.stderr.write(log)
    with open(os.path.join(PKG, "libdock.ptxas.txt"), "w") as f:
        f.write(log)
    os.replace(tmp, LIB)
    with open(STAMP, "w") as f:
        f.write(_defs() + "\n")
    return LIB


if __name__ == "__main__":
    print(build_native(force="--force" in sys.argv, verbose=True))
