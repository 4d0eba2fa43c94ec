"""Build paper_conf_fast_bhatotiarv12_b200/libshred_debug.so: the library with the device-side
bounds checks compiled in (-DSHRED_DEBUG=1, kernels.cuh SHRED_ASSERT).  Run the GPU suite against
it with SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred_debug.so (compute-sanitizer is
closed on the round-2 GPU pool)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_fast_bhatotiarv12_b200 import _build as b  # noqa: E402

print(b.build(out=b.LIB.replace("libshred.so", "libshred_debug.so"), defines=("SHRED_DEBUG=1",)))
