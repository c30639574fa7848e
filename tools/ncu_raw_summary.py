#!/usr/bin/env python
"""Key metrics + stall breakdown from an ncu raw-page CSV export (or a .ncu-rep).

    python tools/ncu_raw_summary.py X.raw.csv|X.ncu-rep [--json]
"""
import csv
import io
import json
import subprocess
import sys

KEYS = ["gpu__time_duration.sum", "launch__registers_per_thread", "launch__grid_size", "launch__block_size",
        "sm__warps_active.avg.pct_of_peak_sustained_active", "smsp__issue_active.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active",
        "sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_lsu.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_uniform.avg.pct_of_peak_sustained_active",
        "smsp__inst_executed.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
        "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed", "dram__throughput.avg.pct_of_peak_sustained_elapsed",
        "sm__cycles_elapsed.avg.per_second", "l1tex__t_requests_pipe_lsu_mem_global_op_ld.sum",
        "l1tex__t_sectors_pipe_lsu_mem_global_op_ld.sum", "lts__t_sectors_srcunit_tex_op_read.sum",
        "l1tex__t_sector_hit_rate.pct", "sm__pipe_tensor_cycles_active_realtime.avg.pct_of_peak_sustained_elapsed",
        "sm__mem_tensor_cycles_active.avg.pct_of_peak_sustained_active"]


def load(path):
    if path.endswith(".csv"):
        text = open(path).read()
    else:
        text = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(text)))
    return rows[0], rows[1], rows[2:]


def summary(path):
    h, u, data = load(path)
    out = []
    for v in data:
        d = dict(zip(h, v))
        units = dict(zip(h, u))
        rec = {"kernel": d.get("Kernel Name", "")[:90]}
        for k in KEYS:
            if k in d:
                rec[k] = f"{d[k]} {units.get(k, '')}".strip()
        st = {}
        for k, x in d.items():
            if k.startswith("smsp__pcsamp_warps_issue_stalled") and not k.endswith("not_issued") and x:
                try:
                    st[k.replace("smsp__pcsamp_warps_issue_stalled_", "")] = float(x.replace(",", ""))
                except ValueError:
                    pass
        tot = sum(st.values()) or 1
        rec["stalls_pct"] = {k: round(100 * x / tot, 1) for k, x in sorted(st.items(), key=lambda t: -t[1])[:10]}
        out.append(rec)
    return out


if __name__ == "__main__":
    s = summary(sys.argv[1])
    if "--json" in sys.argv:
        print(json.dumps(s, indent=1))
    else:
        for rec in s:
            for k, v in rec.items():
                print(f"  {k}: {v}")
