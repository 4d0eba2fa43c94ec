"""B200-native content-defined chunking — the data-parallel hot path of Shredder (FAST'12).

Rabin fingerprint over every 48-byte window (§2.1, §3.1),
cut candidates where fp mod D == r, then the min/max chunk-size rule (L259-L269).
The product is the C-ABI library ``libshred.so`` (include/shred.h, hand-written sm_100a CUDA
in ``csrc/``); this package is its thin Python binding plus the multi-GPU orchestration
(``dist``). See DESIGN.md.
"""
from ._binding import (Chunker, Params, ShredError, synth_fill, lib, LIB_PATH,  # noqa: F401
                       SHRED_PATH_K63, SHRED_PATH_K32, SHRED_PATH_GENERIC)

__all__ = ["Chunker", "Params", "ShredError", "synth_fill", "lib", "LIB_PATH"]
