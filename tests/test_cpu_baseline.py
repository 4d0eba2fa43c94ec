"""The multithreaded CPU chunker baseline agrees with the oracle (so its timing is of the same work)."""
import numpy as np

import cpu_baseline
import oracle
import synthgen


def test_cpu_chunker_matches_oracle():
    data = synthgen.random_bytes(3, (2 << 20) + 77)
    for p in (oracle.Params(), oracle.Params(divisor=256, magic=3),
              oracle.Params(min_size=2048, max_size=65536), oracle.Params(poly=0x104C11DB7, divisor=512)):
        for t in (1, 3, 8):
            got = cpu_baseline.chunk(data, p.poly, p.window, p.divisor, p.magic, p.min_size, p.max_size, t)
            assert np.array_equal(got, oracle.chunk(data, p)), (p, t)
