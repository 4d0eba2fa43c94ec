"""Summarise an ncu --set full report (raw page) for the hot kernel: the counters DESIGN.md cites."""
import csv
import io
import json
import subprocess
import sys

WANT = ['gpu__time_duration.sum', 'dram__bytes_read.sum', 'dram__bytes_write.sum',
        'sm__cycles_elapsed.avg.per_second', 'dram__throughput.avg.pct_of_peak_sustained_elapsed',
        'smsp__issue_active.avg.pct_of_peak_sustained_active', 'smsp__inst_executed.sum',
        'sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active',
        'sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active',
        'sm__inst_executed_pipe_lsu.avg.pct_of_peak_sustained_active',
        'l1tex__data_pipe_lsu_wavefronts_mem_shared.sum', 'l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum',
        'l1tex__data_pipe_lsu_wavefronts.avg.pct_of_peak_sustained_elapsed',
        'l1tex__throughput.avg.pct_of_peak_sustained_active',
        'sm__warps_active.avg.pct_of_peak_sustained_active', 'launch__registers_per_thread',
        'launch__grid_size', 'launch__block_size', 'sm__cycles_active.avg', 'sm__cycles_elapsed.avg',
        'sm__pipe_alu_cycles_active.avg.pct_of_peak_sustained_elapsed']
STALL = 'smsp__average_warps_issue_stalled_'


def summary(rep):
    out = subprocess.run(['ncu', '-i', rep, '--page', 'raw', '--csv'], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    hdr, units, vals = rows[0], rows[1], rows[2]
    d = {}
    for i, h in enumerate(hdr):
        if h in WANT or (h.startswith(STALL) and h.endswith('_per_issue_active.ratio')):
            d[h] = (vals[i], units[i])
    stalls = {k[len(STALL):-len('_per_issue_active.ratio')]: v for k, v in d.items() if k.startswith(STALL)}
    top = sorted(((round(float(v[0].replace(',', '')), 3), k) for k, v in stalls.items()
                  if v[0].replace(',', '').replace('.', '').isdigit()), reverse=True)[:8]
    res = {k: v for k, v in d.items() if k in WANT}
    res['top_stalls'] = top
    try:
        act = float(d['sm__cycles_active.avg'][0].replace(',', ''))
        ela = float(d['sm__cycles_elapsed.avg'][0].replace(',', ''))
        res['sm_active_frac_of_elapsed'] = round(act / ela, 4)
    except (KeyError, ValueError, ZeroDivisionError):
        pass
    return res


if __name__ == '__main__':
    r = summary(sys.argv[1])
    for k, v in r.items():
        print(f'{k:70s} {v}')
