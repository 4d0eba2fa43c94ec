"""Sum gpu__time_duration per kernel name from an ncu --csv launch list (stdin or file)."""
import csv
import sys
from collections import defaultdict

lines = open(sys.argv[1]).read().splitlines() if len(sys.argv) > 1 else sys.stdin.read().splitlines()
i = next(k for k, l in enumerate(lines) if l.startswith('"ID"'))
d = defaultdict(list)
for r in csv.DictReader(lines[i:]):
    if r["Metric Name"] == "gpu__time_duration.sum":
        v = float(r["Metric Value"].replace(",", ""))
        if r["Metric Unit"] == "ns":
            v /= 1e3
        elif r["Metric Unit"] == "ms":
            v *= 1e3
        d[r["Kernel Name"].split("(")[0]].append(v)
for k, v in d.items():
    print(f"{k:60s} n={len(v):4d} mean={sum(v) / len(v):10.2f} us  max={max(v):10.2f} us")
