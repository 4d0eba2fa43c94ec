"""Print an ncu --csv launch list (gpu__time_duration.sum) as `kernel  us` lines.
Usage: ncu --metrics gpu__time_duration.sum --csv ... | python tools/launch_table.py [last_n]"""
import csv
import sys

rows = [r for r in csv.reader(l for l in sys.stdin if l.startswith('"'))]
hdr = rows[0]
ik, im, iv = hdr.index("Kernel Name"), hdr.index("Metric Name"), hdr.index("Metric Value")
out = [(r[ik].split("(")[0][:60], float(r[iv].replace(",", "")) / 1e3) for r in rows[1:]
       if r[im] == "gpu__time_duration.sum"]
n = int(sys.argv[1]) if len(sys.argv) > 1 else len(out)
for k, us in out[-n:]:
    print(f"{k:62s} {us:10.2f} us")
