"""ctypes binding of libshred.so (include/shred.h) — argument marshalling only.

PyTorch supplies device memory, pinned host memory and streams; every step of the chunking
path runs in the library's CUDA kernels. There is no CPU fallback: if libshred.so is missing
or no CUDA device is present, the calls raise.
"""
from __future__ import annotations

import ctypes
import os
from dataclasses import dataclass

import torch

from . import _build

LIB_PATH = os.environ.get("SHRED_LIB", _build.LIB)   # override: A/B variant builds

SHRED_PATH_K63, SHRED_PATH_K32, SHRED_PATH_GENERIC = 1, 2, 3
PATH_NAMES = {1: "k63", 2: "k32", 3: "generic"}


class ShredError(RuntimeError):
    pass


class _Params(ctypes.Structure):
    _fields_ = [("poly", ctypes.c_uint64), ("window", ctypes.c_uint32), ("marker", ctypes.c_uint32),
                ("divisor", ctypes.c_uint64), ("magic", ctypes.c_uint64),
                ("min_size", ctypes.c_uint64), ("max_size", ctypes.c_uint64)]


class _HashJob(ctypes.Structure):
    _fields_ = [("d_in", ctypes.c_void_p), ("len", ctypes.c_uint64), ("d_cuts", ctypes.c_void_p),
                ("d_ncuts", ctypes.c_void_p), ("d_digests", ctypes.c_void_p), ("max_chunks", ctypes.c_uint64)]


@dataclass(frozen=True)
class Params:
    """shred_params. Defaults = the paper's readings (Q1, Q5, Q6, Q15)."""
    poly: int = 0xBFE6B8A5BF378D83
    window: int = 48
    divisor: int = 8192
    magic: int = 0x78
    min_size: int = 0
    max_size: int = 0
    marker: int = 0          # 0: fp mod D == r (L447-L451); 1: fp mod D <= r (L249-L251)

    def _c(self) -> _Params:
        return _Params(self.poly, self.window, self.marker, self.divisor, self.magic, self.min_size,
                       self.max_size)


_lib = None


def lib() -> ctypes.CDLL:
    """Load libshred.so (building it in-tree if the sources are newer). Raises if unavailable."""
    global _lib
    if _lib is None:
        if LIB_PATH == _build.LIB and _build.stale():
            _build.build()
        if not os.path.exists(LIB_PATH):
            raise ShredError(f"{LIB_PATH} missing: run __graft_entry__.build()")
        L = ctypes.CDLL(LIB_PATH)
        u64, u32, cint, vp = ctypes.c_uint64, ctypes.c_uint32, ctypes.c_int, ctypes.c_void_p
        P = ctypes.POINTER(_Params)
        sig = {
            "shred_default_params": (None, [P]),
            "shred_init": (cint, [P, cint, ctypes.POINTER(vp)]),
            "shred_destroy": (None, [vp]),
            "shred_strerror": (ctypes.c_char_p, [cint]),
            "shred_last_error": (ctypes.c_char_p, [vp]),
            "shred_path": (cint, [vp]),
            "shred_kernel_mode": (cint, [vp]),
            "shred_get_params": (cint, [vp, P]),
            "shred_max_cuts": (u64, [vp, u64]),
            "shred_chunk": (cint, [vp, vp, u64, vp, u64, vp, vp]),
            "shred_candidates_range": (cint, [vp, vp, u64, u64, u64, u64, vp, u64, vp, vp]),
            "shred_size_bound": (cint, [vp, vp, u64, u64, vp, u64, vp, vp]),
            "shred_feed": (cint, [vp, vp, u64, vp, u64, vp, vp]),
            "shred_flush": (cint, [vp, vp, u64, vp, vp]),
            "shred_reset": (cint, [vp]),
            "shred_set_ring": (cint, [vp, cint, u64]),
            "shred_synth_fill": (cint, [vp, u64, u64, u64, vp]),
            "shred_launch_count": (u64, [vp]),
            "shred_hash_chunks": (cint, [vp, vp, u64, vp, vp, vp, u64, vp]),
            "shred_index_reset": (cint, [vp, u64]),
            "shred_hash_chunks_batch": (cint, [vp, vp, cint, vp]),
            "shred_size_bound_state": (cint, [vp, vp, u64, u64, cint, ctypes.POINTER(u64), vp, u64, vp, vp, vp]),
            "shred_size_bound_state_dev": (cint, [vp, vp, vp, u64, u64, cint, vp, vp, u64, vp, vp, vp]),
            "shred_index_insert": (cint, [vp, vp, vp, vp, u64, u64, vp, vp]),
            "shred_index_stats": (cint, [vp, ctypes.POINTER(u64)]),
            "shred_profile": (cint, [vp, cint]),
            "shred_profile_read": (cint, [vp, ctypes.POINTER(ctypes.c_double), ctypes.POINTER(u64),
                                          ctypes.POINTER(u64)]),
        }
        for name, (res, args) in sig.items():
            fn = getattr(L, name, None)
            if fn is None:                      # an older A/B build (SHRED_LIB) without this call
                continue
            fn.restype = res
            fn.argtypes = args
        _lib = L
    return _lib


_raw_stream = getattr(torch._C, "_cuda_getCurrentRawStream", None)


def _stream(stream) -> int:
    if stream is None:
        # the current stream's cudaStream_t without building a torch.cuda.Stream object (~2 us)
        if _raw_stream is not None:
            return _raw_stream(torch.cuda.current_device())
        return torch.cuda.current_stream().cuda_stream
    if isinstance(stream, torch.cuda.Stream):
        return stream.cuda_stream
    return int(stream)


def synth_fill(buf: torch.Tensor, seed: int, offset: int = 0, stream=None) -> None:
    """Fill a CUDA uint8 tensor with bytes [offset, offset+n) of SplitMix64 stream `seed`."""
    assert buf.is_cuda and buf.dtype == torch.uint8 and buf.is_contiguous()
    rc = lib().shred_synth_fill(buf.data_ptr(), buf.numel(), seed, offset, _stream(stream))
    if rc:
        raise ShredError(f"shred_synth_fill: {rc}")


class Chunker:
    """One shred_ctx: a chunker bound to one CUDA device with fixed parameters."""

    def __init__(self, params: Params = Params(), device: int | None = None):
        if not torch.cuda.is_available():
            raise ShredError("no CUDA device: the chunker has no CPU fallback")
        self.params = params
        self.device = torch.cuda.current_device() if device is None else int(device)
        self._ctx = ctypes.c_void_p()
        cp = params._c()
        rc = lib().shred_init(ctypes.byref(cp), self.device, ctypes.byref(self._ctx))
        if rc:
            raise ShredError(f"shred_init: {lib().shred_strerror(rc).decode()} ({rc}) for {params}")
        dev = torch.device("cuda", self.device)
        self._n = torch.zeros(1, dtype=torch.int64, device=dev)
        self._chunk = lib().shred_chunk          # bound once: the per-call path is argument marshalling only

    def close(self):
        if self._ctx:
            lib().shred_destroy(self._ctx)
            self._ctx = ctypes.c_void_p()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def _check(self, rc: int, what: str):
        if rc:
            detail = lib().shred_last_error(self._ctx).decode()
            raise ShredError(f"{what}: {lib().shred_strerror(rc).decode()} ({rc}): {detail}")

    @property
    def path(self) -> str:
        return PATH_NAMES.get(lib().shred_path(self._ctx), "?")

    @property
    def mode(self) -> str:
        """The hot kernel's state mode (k63, k40, k63t, k32, k32b, k32t, generic)."""
        return {1: "k63", 2: "k32", 3: "generic", 4: "k32b", 5: "k40", 6: "k32t", 7: "k63t"}.get(
            lib().shred_kernel_mode(self._ctx), "?")

    @property
    def launches(self) -> int:
        return int(lib().shred_launch_count(self._ctx))

    def profile(self, enable: bool) -> None:
        self._check(lib().shred_profile(self._ctx, int(enable)), "shred_profile")

    def profile_read(self) -> tuple[float, int, int]:
        """(summed ms, launches, input bytes) of the hot kernel since the last read."""
        ms, n, b = ctypes.c_double(), ctypes.c_uint64(), ctypes.c_uint64()
        self._check(lib().shred_profile_read(self._ctx, ctypes.byref(ms), ctypes.byref(n), ctypes.byref(b)),
                    "shred_profile_read")
        return ms.value, n.value, b.value

    def max_cuts(self, n: int) -> int:
        return int(lib().shred_max_cuts(self._ctx, n))

    def _out(self, cap: int) -> torch.Tensor:
        return torch.empty(max(1, cap), dtype=torch.int64, device=torch.device("cuda", self.device))

    # ---------------------------------------------------------------- one-shot
    def chunk_async(self, x: torch.Tensor, out: torch.Tensor, n_out: torch.Tensor, stream=None) -> None:
        """Enqueue shred_chunk; out (int64) gets the cuts, n_out[0] the true count."""
        if x.dtype != torch.uint8 or not x.is_cuda or not x.is_contiguous():
            raise ShredError("shred_chunk: x must be a contiguous CUDA uint8 tensor")
        rc = self._chunk(self._ctx, x.data_ptr(), x.numel(), out.data_ptr(), out.numel(),
                         n_out.data_ptr(), _stream(stream))
        if rc:
            self._check(rc, "shred_chunk")

    def _guess(self, n: int) -> int:
        return min(self.max_cuts(n), n // 512 + 4096) if n > 1 else 1

    def chunk(self, x: torch.Tensor, cap: int | None = None) -> torch.Tensor:
        """Final cut offsets of the device-resident stream x (synchronises; re-runs once with
        the exact capacity if the first guess was too small)."""
        c = self._guess(x.numel()) if cap is None else cap
        out = self._out(c)
        self.chunk_async(x, out, self._n)
        n = int(self._n.item())
        if n > c:
            if cap is not None:
                raise ShredError(f"capacity {cap} < {n} cuts")
            out = self._out(n)
            self.chunk_async(x, out, self._n)
            n = int(self._n.item())
        return out[:n]

    def candidates_range(self, x: torch.Tensor, halo: int, start: int, total_len: int,
                         cap: int | None = None) -> torch.Tensor:
        """Candidates of window ends [start, start + len(x) - halo) of a stream of total_len."""
        assert x.is_cuda and x.dtype == torch.uint8 and x.is_contiguous()
        ln = x.numel() - halo
        c = self._guess(ln + 1) if cap is None else cap
        for _ in range(2):
            out = self._out(c)
            rc = lib().shred_candidates_range(self._ctx, x.data_ptr(), halo, start, ln, total_len,
                                              out.data_ptr(), out.numel(), self._n.data_ptr(), _stream(None))
            self._check(rc, "shred_candidates_range")
            n = int(self._n.item())
            if n <= c:
                return out[:n]
            if cap is not None:
                break
            c = n
        raise ShredError(f"capacity {c} < {n} candidates")

    def _rule_cap(self, n_cand: int, span: int) -> int:
        """Cuts the size rule can emit over `span` bytes from `n_cand` candidates: the accepted
        candidates, the forced cuts (one per max_size bytes) and a held cut; with min_size > 0
        also at most span // min_size + 1 (bounded by the range, not by its
        absolute end offset)."""
        p = self.params
        cap = n_cand + (span // p.max_size + 1 if p.max_size else 0) + 2
        if p.min_size:
            cap = min(cap, span // p.min_size + 2)
        return max(1, cap)

    def candidates_range_async(self, x: torch.Tensor, halo: int, start: int, total_len: int,
                               out: torch.Tensor, n_out: torch.Tensor, stream=None) -> None:
        """Enqueue shred_candidates_range; no host synchronisation (n_out[0] = the true count,
        min(count, len(out)) offsets written)."""
        assert x.is_cuda and x.dtype == torch.uint8 and x.is_contiguous()
        rc = lib().shred_candidates_range(self._ctx, x.data_ptr(), halo, start, x.numel() - halo, total_len,
                                          out.data_ptr(), out.numel(), n_out.data_ptr(), _stream(stream))
        self._check(rc, "shred_candidates_range")

    def size_bound_state_dev(self, cands: torch.Tensor, n_cand: torch.Tensor, end: int, fin: bool,
                             state_in: torch.Tensor, out: torch.Tensor, n_out: torch.Tensor,
                             state_out: torch.Tensor, stream=None) -> None:
        """Enqueue shred_size_bound_state_dev: the candidate count (n_cand[0], clamped to
        len(cands)) and the entry state {s, held} (state_in) are device values; exit state to
        state_out.  No host synchronisation."""
        for t in (cands, n_cand, state_in, out, n_out, state_out):
            assert t.is_cuda and t.dtype == torch.int64 and t.is_contiguous()
        rc = lib().shred_size_bound_state_dev(self._ctx, cands.data_ptr(), n_cand.data_ptr(), cands.numel(), end,
                                              int(fin), state_in.data_ptr(), out.data_ptr(), out.numel(),
                                              n_out.data_ptr(), state_out.data_ptr(), _stream(stream))
        self._check(rc, "shred_size_bound_state_dev")

    def size_bound(self, cands: torch.Tensor, total_len: int, cap: int | None = None) -> torch.Tensor:
        assert cands.is_cuda and cands.dtype == torch.int64 and cands.is_contiguous()
        cap = self._rule_cap(cands.numel(), total_len) if cap is None else cap
        out = self._out(cap)
        rc = lib().shred_size_bound(self._ctx, cands.data_ptr(), cands.numel(), total_len,
                                    out.data_ptr(), out.numel(), self._n.data_ptr(), _stream(None))
        self._check(rc, "shred_size_bound")
        n = int(self._n.item())
        if n > cap:
            raise ShredError(f"capacity {cap} < {n} cuts")
        return out[:n]

    def size_bound_state(self, cands: torch.Tensor, end: int, fin: bool, s: int, held: bool,
                         cap: int | None = None) -> tuple[torch.Tensor, int, bool]:
        """The size rule over one stream range from entry state (s, held): (cuts, exit s, exit held)."""
        assert cands.dtype == torch.int64 and cands.is_contiguous()
        dev = torch.device("cuda", self.device)
        c = cands if cands.is_cuda else cands.to(dev)
        cap = self._rule_cap(c.numel(), end - s) if cap is None else cap
        out = self._out(cap)
        st = torch.zeros(2, dtype=torch.int64, device=dev)
        sin = (ctypes.c_uint64 * 2)(s, int(held))
        rc = lib().shred_size_bound_state(self._ctx, c.data_ptr() if c.numel() else None, c.numel(), end, int(fin),
                                          sin, out.data_ptr(), out.numel(), self._n.data_ptr(), st.data_ptr(),
                                          _stream(None))
        self._check(rc, "shred_size_bound_state")
        n = int(self._n.item())
        if n > cap:
            raise ShredError(f"capacity {cap} < {n} cuts")
        sv = st.cpu().tolist()
        return out[:n], int(sv[0]), bool(sv[1])

    # ---------------------------------------------------------------- hashing (f2)
    def hash_chunks_async(self, x: torch.Tensor, cuts: torch.Tensor, n_cuts: torch.Tensor,
                          digests: torch.Tensor, stream=None) -> None:
        """Enqueue SHA-256 of every chunk delimited by cuts[:n_cuts[0]] (device count)."""
        assert x.is_cuda and x.dtype == torch.uint8 and x.is_contiguous()
        assert digests.dtype == torch.uint8 and digests.is_contiguous() and digests.numel() % 32 == 0
        rc = lib().shred_hash_chunks(self._ctx, x.data_ptr(), x.numel(), cuts.data_ptr(), n_cuts.data_ptr(),
                                     digests.data_ptr(), digests.numel() // 32, _stream(stream))
        self._check(rc, "shred_hash_chunks")

    def hash_chunks_batch_async(self, jobs, stream=None) -> None:
        """Enqueue shred_hash_chunks_batch: jobs = [(x, cuts, n_cuts, digests), ...] as in
        hash_chunks_async; one length-sorted work list over every buffer's chunks."""
        arr = (_HashJob * len(jobs))()
        for k, (x, cuts, n_cuts, digests) in enumerate(jobs):
            assert x.is_cuda and x.dtype == torch.uint8 and x.is_contiguous()
            assert digests.dtype == torch.uint8 and digests.is_contiguous() and digests.numel() % 32 == 0
            arr[k] = _HashJob(x.data_ptr(), x.numel(), cuts.data_ptr(), n_cuts.data_ptr(), digests.data_ptr(),
                              digests.numel() // 32)
        rc = lib().shred_hash_chunks_batch(self._ctx, ctypes.cast(arr, ctypes.c_void_p), len(jobs), _stream(stream))
        self._check(rc, "shred_hash_chunks_batch")

    def hash_chunks(self, x: torch.Tensor, cuts: torch.Tensor) -> torch.Tensor:
        """(len(cuts)+1, 32) uint8 SHA-256 digests of the chunks of x (synchronises)."""
        n = torch.tensor([cuts.numel()], dtype=torch.int64, device=x.device)
        out = torch.empty((cuts.numel() + 1) * 32 if x.numel() else 32, dtype=torch.uint8, device=x.device)
        c = cuts.contiguous() if cuts.numel() else torch.zeros(1, dtype=torch.int64, device=x.device)
        self.hash_chunks_async(x, c, n, out)
        torch.cuda.current_stream().synchronize()
        return out.view(-1, 32)[: (cuts.numel() + 1) if x.numel() else 0]

    # ---------------------------------------------------------------- dedup index (f3)
    def index_reset(self, capacity: int) -> None:
        self._check(lib().shred_index_reset(self._ctx, capacity), "shred_index_reset")

    def index_insert_async(self, digests: torch.Tensor, cuts: torch.Tensor, n_cuts: torch.Tensor, length: int,
                           new_flags: torch.Tensor | None = None, stream=None) -> None:
        assert digests.dtype == torch.uint8 and digests.is_contiguous()
        rc = lib().shred_index_insert(self._ctx, digests.data_ptr(), cuts.data_ptr(), n_cuts.data_ptr(), length,
                                      digests.numel() // 32,
                                      new_flags.data_ptr() if new_flags is not None else None, _stream(stream))
        self._check(rc, "shred_index_insert")

    def index_stats(self) -> dict:
        arr = (ctypes.c_uint64 * 4)()
        self._check(lib().shred_index_stats(self._ctx, arr), "shred_index_stats")
        return {"chunks": arr[0], "new_chunks": arr[1], "new_bytes": arr[2], "full": arr[3]}

    # ---------------------------------------------------------------- streaming
    def feed_async(self, x: torch.Tensor, out: torch.Tensor, n_out: torch.Tensor, stream=None) -> None:
        assert x.dtype == torch.uint8 and x.is_contiguous()
        assert x.numel() == 0 or x.is_cuda or x.is_pinned(), "host input must be pinned"
        rc = lib().shred_feed(self._ctx, x.data_ptr(), x.numel(), out.data_ptr(), out.numel(),
                              n_out.data_ptr(), _stream(stream))
        self._check(rc, "shred_feed")

    def feed(self, x: torch.Tensor, cap: int | None = None) -> torch.Tensor:
        """Feed one buffer (device or pinned host); returns its final cuts (synchronises).
        The default capacity cannot overflow (a streaming overflow is sticky)."""
        cap = self.max_cuts(x.numel() + 2) + 1 if cap is None else cap
        out = self._out(cap)
        self.feed_async(x, out, self._n)
        n = int(self._n.item())
        if n > cap:
            raise ShredError(f"capacity {cap} < {n} cuts")
        return out[:n]

    def flush(self, cap: int = 64) -> torch.Tensor:
        """End the stream; returns the cuts it emits (the feeds have already emitted every cut
        strictly inside the stream that they could decide, so this is normally empty)."""
        out = self._out(cap)
        rc = lib().shred_flush(self._ctx, out.data_ptr(), out.numel(), self._n.data_ptr(), _stream(None))
        self._check(rc, "shred_flush")
        n = int(self._n.item())
        if n > cap:
            raise ShredError(f"capacity {cap} < {n} cuts")
        return out[:n]

    def reset(self) -> None:
        self._check(lib().shred_reset(self._ctx), "shred_reset")

    def set_ring(self, slots: int, slot_bytes: int) -> None:
        self._check(lib().shred_set_ring(self._ctx, slots, slot_bytes), "shred_set_ring")
