"""profiles/k1_traffic.json from an ncu --set full capture of k1_bulk (the `traffic` field of
bench.py's roofline): dram__bytes_read.sum + dram__bytes_write.sum of the captured launch.

Usage: python tools/ncu_traffic.py <report.ncu-rep> <summary-file-it-is-committed-as> > profiles/k1_traffic.json
gpu_profile.sh writes the summary text and this JSON from the same report in one run, so the
number bench.py prints is the one in the committed summary."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
from ncu_summary import summary  # noqa: E402


def num(v):
    return float(str(v[0]).replace(",", ""))


def scale(v):
    u = v[1].strip().lower()
    return {"byte": 1, "kbyte": 1e3, "mbyte": 1e6, "gbyte": 1e9}.get(u, 1)


def main():
    rep, cited = sys.argv[1], sys.argv[2]
    s = summary(rep)
    rd = num(s["dram__bytes_read.sum"]) * scale(s["dram__bytes_read.sum"])
    wr = num(s["dram__bytes_write.sum"]) * scale(s["dram__bytes_write.sum"])
    print(json.dumps({"kernel": "k1_bulk (the bench's hot kernel)", "source": cited,
                      "report": os.path.basename(rep),
                      "dram_bytes_per_launch": int(round(rd + wr)),
                      "dram_bytes_read": int(round(rd)), "dram_bytes_write": int(round(wr)),
                      "grid": s.get("launch__grid_size", ["?"])[0], "block": s.get("launch__block_size", ["?"])[0],
                      "duration": s.get("gpu__time_duration.sum")}, indent=1))


if __name__ == "__main__":
    main()
