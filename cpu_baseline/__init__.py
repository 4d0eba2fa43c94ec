"""Multithreaded CPU rolling chunker (§5.1): a timed baseline, not the oracle.

Built with gcc -O3 -march=x86-64-v3 -pthread into cpu_baseline/libcpuchunk.so.  Only bench.py and
tests use it."""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "cpu_chunker.c")
_LIB = os.path.join(_HERE, "libcpuchunk.so")
_lib = None


def build(force: bool = False) -> str:
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O3", "-march=x86-64-v3", "-std=c11", "-fPIC", "-shared", "-pthread",
                               "-o", tmp, _SRC])
        os.replace(tmp, _LIB)
    return _LIB


def chunk(data: np.ndarray, poly=0xBFE6B8A5BF378D83, window=48, divisor=8192, magic=0x78,
          min_size=0, max_size=0, threads: int | None = None) -> np.ndarray:
    global _lib
    if _lib is None:
        build()
        _lib = ctypes.CDLL(_LIB)
        u64 = ctypes.c_uint64
        _lib.cpu_chunk.restype = ctypes.c_int64
        _lib.cpu_chunk.argtypes = [ctypes.c_void_p, u64, u64, ctypes.c_uint32, u64, u64, u64, u64,
                                   ctypes.c_int, ctypes.c_void_p, u64]
    a = np.ascontiguousarray(data, dtype=np.uint8)
    threads = threads or len(os.sched_getaffinity(0))
    cap = a.size // 1024 + 65536
    while True:
        out = np.zeros(cap, dtype=np.uint64)
        n = _lib.cpu_chunk(a.ctypes.data, a.size, poly, window, divisor, magic, min_size, max_size,
                           threads, out.ctypes.data, cap)
        if n <= cap:
            return out[:n]
        cap = int(n)
