"""C-ABI library: it builds for sm_100a, loads, and exports every symbol include/shred.h declares.
No compute calls (no GPU here)."""
import ctypes
import os
import re
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "shred.h")


def declared_functions():
    src = open(HEADER).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(shred_[a-z0-9_]+)\s*\(", src)))


@pytest.fixture(scope="module")
def libpath():
    from paper_conf_fast_bhatotiarv12_b200 import _build
    return _build.build()


def test_header_declares_the_boundary():
    names = declared_functions()
    for must in ("shred_init", "shred_chunk", "shred_feed", "shred_flush", "shred_destroy",
                 "shred_default_params", "shred_candidates_range", "shred_size_bound"):
        assert must in names


def test_library_exports_every_declared_symbol(libpath):
    out = subprocess.run(["nm", "-D", "--defined-only", libpath], capture_output=True, text=True).stdout
    exported = set(re.findall(r"\bT (shred_\w+)", out))
    missing = [n for n in declared_functions() if n not in exported]
    assert not missing, missing
    L = ctypes.CDLL(libpath)
    for n in declared_functions():
        assert getattr(L, n) is not None


def test_library_is_sm100a_only(libpath):
    out = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "--list-elf", libpath],
                         capture_output=True, text=True).stdout
    assert "sm_100a" in out
    for other in ("sm_90", "sm_80", "sm_103"):
        assert other not in out


def test_hot_kernel_uses_tma(libpath):
    sass = subprocess.run(["/usr/local/cuda/bin/cuobjdump", "-sass", libpath],
                          capture_output=True, text=True).stdout
    assert "UTMALDG" in sass       # cp.async.bulk.tensor (TMA) in k1_bulk


def test_default_params_and_strerror_without_gpu(libpath):
    from paper_conf_fast_bhatotiarv12_b200._binding import _Params, lib
    p = _Params()
    lib().shred_default_params(ctypes.byref(p))
    assert p.poly == 0xBFE6B8A5BF378D83 and p.window == 48 and p.divisor == 8192 and p.magic == 0x78
    assert p.min_size == 0 and p.max_size == 0
    assert lib().shred_strerror(-1) == b"invalid argument"


def test_init_rejects_bad_params_without_touching_the_gpu(libpath):
    from paper_conf_fast_bhatotiarv12_b200._binding import _Params, lib
    ctx = ctypes.c_void_p()
    bad = [
        _Params((1 << 63) | 1, 48, 0, 8192, 0x78, 0, 0),          # reducible x^63+1
        _Params(0xBFE6B8A5BF378D83, 0, 0, 8192, 0x78, 0, 0),      # w = 0
        _Params(0xBFE6B8A5BF378D83, 48, 2, 8192, 0x78, 0, 0),     # unknown marker mode
        _Params(0xBFE6B8A5BF378D83, 48, 0, 1, 0, 0, 0),           # D < 2
        _Params(0xBFE6B8A5BF378D83, 48, 0, 8192, 8192, 0, 0),     # r >= D
        _Params(0xBFE6B8A5BF378D83, 48, 0, 8192, 0x78, 100, 50),  # max < min
        _Params(0x1F, 48, 0, 4, 0, 0, 0),                         # degree 4 < 8
    ]
    for p in bad:
        assert lib().shred_init(ctypes.byref(p), 0, ctypes.byref(ctx)) == -1
        assert not ctx.value
