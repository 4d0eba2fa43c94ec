"""In-tree build of libshred.so (nvcc, sm_100a only). Used by __graft_entry__.build().

shred.cu (host side, C ABI, the other kernels) and the hot kernel's instances (k1_inst.cu, one
object per state mode) compile as separate objects in parallel, then link into one shared
library with the CUDA runtime linked statically.
"""
from __future__ import annotations

import os
import shutil
import subprocess
import tempfile

PKG = os.path.dirname(os.path.abspath(__file__))
CSRC = os.path.join(PKG, "csrc")
LIB = os.path.join(PKG, "libshred.so")
SOURCES = [os.path.join(CSRC, "shred.cu"), os.path.join(CSRC, "k1_inst.cu")]
DEPS = SOURCES + [os.path.join(CSRC, f) for f in ("kernels.cuh", "size_bound.cuh", "sha256.cuh", "dedup.cuh")] + \
       [os.path.join(os.path.dirname(PKG), "include", "shred.h")]
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")
CFLAGS = ["-O3", "-std=c++17", "-lineinfo", "-gencode", "arch=compute_100a,code=sm_100a",
          "-Xcompiler", "-fPIC,-O2", "--expt-relaxed-constexpr", "-Xptxas", "-v"]
# object -> (source, extra defines); SHRED_INST = kernels.cuh MODE_* (K63 1, K32 2, K32B 4, K40 5, K32T 6, K63T 7)
UNITS = [("shred", "shred.cu", ()), ("k1_sel", "k1_inst.cu", ("SHRED_INST=0",)),
         ("k1_k63", "k1_inst.cu", ("SHRED_INST=1",)), ("k1_k32", "k1_inst.cu", ("SHRED_INST=2",)),
         ("k1_k32b", "k1_inst.cu", ("SHRED_INST=4",)), ("k1_k40", "k1_inst.cu", ("SHRED_INST=5",)),
         ("k1_k32t", "k1_inst.cu", ("SHRED_INST=6",)), ("k1_k63t", "k1_inst.cu", ("SHRED_INST=7",))]


def stale() -> bool:
    if not os.path.exists(LIB):
        return True
    t = os.path.getmtime(LIB)
    return any(os.path.getmtime(d) > t for d in DEPS)


def build(force: bool = False, verbose: bool = False, out: str | None = None,
          defines: tuple[str, ...] = ()) -> str:
    """Build libshred.so (or a variant `out` with extra -D defines, for A/B measurements)."""
    target = out or LIB
    if out is None and not force and not stale():
        return LIB
    tmpdir = tempfile.mkdtemp(prefix="shred_build_")
    try:
        procs = []
        for name, src, defs in UNITS:
            obj = os.path.join(tmpdir, name + ".o")
            cmd = [NVCC, *CFLAGS, *[f"-D{d}" for d in (*defs, *defines)], "-c", "-o", obj,
                   os.path.join(CSRC, src)]
            procs.append((obj, subprocess.Popen(cmd, stdout=subprocess.PIPE, stderr=subprocess.PIPE, text=True)))
        logs, objs = [], []
        for obj, p in procs:
            so, se = p.communicate()
            if p.returncode != 0:
                raise RuntimeError("nvcc failed:\n" + so + se)
            logs.append(se)
            objs.append(obj)
        tmp = target + f".tmp{os.getpid()}"
        r = subprocess.run([NVCC, "-shared", "-cudart", "static", "-gencode", "arch=compute_100a,code=sm_100a",
                            "-o", tmp, *objs], capture_output=True, text=True)
        if r.returncode != 0:
            raise RuntimeError("nvcc link failed:\n" + r.stdout + r.stderr)
    finally:
        shutil.rmtree(tmpdir, ignore_errors=True)
    if verbose:
        print("".join(logs))
    if out is None:
        with open(os.path.join(PKG, "ptxas_info.txt"), "w") as f:
            f.write("".join(logs))
    os.replace(tmp, target)
    return target


if __name__ == "__main__":
    build(force=True, verbose=True)
