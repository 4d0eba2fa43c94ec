"""In-tree build of libshred.so (nvcc, sm_100a only). Used by __graft_entry__.build()."""
from __future__ import annotations

import os
import subprocess

PKG = os.path.dirname(os.path.abspath(__file__))
CSRC = os.path.join(PKG, "csrc")
LIB = os.path.join(PKG, "libshred.so")
SOURCES = [os.path.join(CSRC, "shred.cu")]
DEPS = SOURCES + [os.path.join(CSRC, "kernels.cuh"),
                  os.path.join(os.path.dirname(PKG), "include", "shred.h")]
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")
FLAGS = ["-O3", "-std=c++17", "-lineinfo", "-gencode", "arch=compute_100a,code=sm_100a",
         "-Xcompiler", "-fPIC,-O2", "-shared", "-cudart", "static", "--expt-relaxed-constexpr",
         "-Xptxas", "-v"]


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
    tmp = target + f".tmp{os.getpid()}"
    cmd = [NVCC, *FLAGS, *[f"-D{d}" for d in defines], "-o", tmp, *SOURCES]
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        raise RuntimeError("nvcc failed:\n" + r.stdout + r.stderr)
    if verbose:
        print(r.stderr)
    if out is None:
        with open(os.path.join(PKG, "ptxas_info.txt"), "w") as f:
            f.write(r.stderr)
    os.replace(tmp, target)
    return target


if __name__ == "__main__":
    build(force=True, verbose=True)
