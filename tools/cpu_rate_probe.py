"""Why the oracle's host rate differs between bench arms: the same R2 oracle
on differently produced / sized samples, fresh process, all cores.  Prints one line per case."""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402

import oracle  # noqa: E402
import synthgen  # noqa: E402

oracle.build()
cores = len(os.sched_getaffinity(0))


def rate(a, reps=3):
    r = []
    for _ in range(reps):
        t = time.perf_counter()
        oracle.candidates(a, oracle.Params(), 2, cores)
        r.append(a.size / (time.perf_counter() - t) / 1e9)
    return " ".join(f"{x:.3f}" for x in r)


print("cores", cores, "numa", os.popen("lscpu | grep -i numa").read().replace("\n", " | "))
a = synthgen.random_bytes(2, 256 << 20)
print("numpy-gen 256 MiB", rate(a))
b = synthgen.random_bytes_fast(2, 256 << 20)
print("fast-gen 256 MiB ", rate(b))
c = synthgen.random_bytes_fast(2, 1 << 30)
print("fast-gen 1 GiB   ", rate(c))
print("fast-gen 1 GiB, 256 MiB slice", rate(c[: 256 << 20]))
d = np.empty(1 << 30, np.uint8)
synthgen.fill_fast(d, 2, 0, threads=1)
print("1-thread fill 1 GiB", rate(d))
