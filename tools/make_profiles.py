#!/usr/bin/env python
"""Turn one measurement batch (tools/gpu_round.sh output in gpurun_out/) into the committed evidence
under profiles/:

    profiles/<tag>_bench.json             the bench.py JSON line
    profiles/<tag>_launches.csv           ncu launch list of `bench.py --steps 2 --warmup 3` (our kernels)
    profiles/<tag>_launch_shares.txt      per-kernel share of the timed steps (cold-cache, serialised)
    profiles/<tag>_ncu_<name>.txt         ncu --set full summaries (key metrics + stall breakdown)
    profiles/ncu_traffic.json             dram bytes (read + write) per launch, by bench point name

    python tools/make_profiles.py <tag> [gpurun_out]
"""
import csv
import io
import json
import os
import re
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, os.path.join(ROOT, "tools"))
import ncu_raw_summary  # noqa: E402

def dram_bytes(v: str) -> float:
    """'1.502640 Gbyte' -> bytes (each metric carries its own unit)."""
    num, unit = v.split()[:2]
    return float(num.replace(",", "")) * {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}[unit]


# ncu capture name -> bench point name (tools/gpu_round.sh profiles these configurations)
CAPTURES = {
    "prof_k15_b8_s8192": "conv2d_single 8192^2 K=15 x8 images",
    "prof_k3_b8_s8192": "conv2d_single 8192^2 K=3 x8 images",
    "prof_k7_b8_s8192": "conv2d_single 8192^2 K=7 x8 images",
    "prof_k15_v0_s8192": "conv2d_single 8192^2 K=15",
    "prof_k3_v0_s8192": "conv2d_single 8192^2 K=3",
    "prof_k7_v0_s8192": "conv2d_single 8192^2 K=7",
    "prof_k15_s4096": "conv2d_single 4096^2 K=15",
    "prof_k5_s2048": "conv2d_single 2048^2 K=5",
    "prof_direct_k3_s8192": "conv2d_single_direct 8192^2 K=3 (Fig. 1a baseline)",
    "prof_tc_config2": "conv2d_multi_tc N32 C64 F64 56^2 K3",
    "prof_tc_config3": "conv2d_multi_tc N128 C3 F64 224^2 K7",
    "prof_multi_config3": "conv2d_multi N128 C3 F64 224^2 K7",
    "prof_split_k15_s1024": "conv2d_single 1024^2 K=15 (filter-row split, cluster of 2 CTAs)",
    "prof_conv11c1": "conv2d_multi Table I CONV11 C1 N128 224^2 F64 K3",
    "prof_config0": "conv2d_single 256^2 K=3 (configs[0], one image)",
}


def launches(path, out_csv, out_txt):
    text = open(path).read()
    lines = [ln for ln in text.splitlines() if ln.startswith('"')]
    rows = list(csv.reader(io.StringIO("\n".join(lines))))
    hdr = rows[0]
    ik, iv, ig = hdr.index("Kernel Name"), hdr.index("Metric Value"), hdr.index("Grid Size")
    ours = [(r[ik], r[ig], float(r[iv].replace(",", ""))) for r in rows[1:] if "conv2d" in r[ik]]
    with open(out_csv, "w") as fh:
        w = csv.writer(fh)
        w.writerow(["kernel", "grid", "gpu__time_duration.sum (ns)"])
        for k, g, t in ours:
            w.writerow([k, g, t])
    # the last 2 steps of 28 launches are the timed ones
    timed = ours[-56:] if len(ours) >= 56 else ours
    tot = sum(t for _, _, t in timed)
    by = {}
    for k, g, t in timed:
        key = re.sub(r"\s+", " ", k)
        by.setdefault((key, g), []).append(t)
    with open(out_txt, "w") as fh:
        fh.write(f"ncu launch list (cold-cache, serialised): {len(timed)} launches of 2 timed steps, "
                 f"total {tot / 1e3:.1f} us\n")
        for (k, g), ts in sorted(by.items(), key=lambda kv: -sum(kv[1])):
            fh.write(f"{100 * sum(ts) / tot:6.2f}%  {sum(ts) / len(ts) / 1e3:9.2f} us/launch  x{len(ts)}  grid {g}  {k}\n")


def main():
    tag = sys.argv[1]
    src = sys.argv[2] if len(sys.argv) > 2 else os.path.join(ROOT, "gpurun_out")
    dst = os.path.join(ROOT, "profiles")
    os.makedirs(dst, exist_ok=True)
    b = os.path.join(src, f"bench_{tag}.json")
    if os.path.exists(b):
        line = open(b).read().strip().splitlines()[-1]
        json.loads(line)
        open(os.path.join(dst, f"{tag}_bench.json"), "w").write(line + "\n")
    for f in sorted(os.listdir(src)):  # the other workloads' bench lines
        m = re.fullmatch(rf"bench_{re.escape(tag)}_(\w+)\.json", f)
        if m:
            lines = open(os.path.join(src, f)).read().strip().splitlines()
            if lines:
                try:
                    json.loads(lines[-1])
                except ValueError:
                    continue
                open(os.path.join(dst, f"{tag}_bench_{m.group(1)}.json"), "w").write(lines[-1] + "\n")
    lfile = os.path.join(src, f"launches_{tag}.csv")
    if os.path.exists(lfile):
        launches(lfile, os.path.join(dst, f"{tag}_launches.csv"), os.path.join(dst, f"{tag}_launch_shares.txt"))
    traffic_path = os.path.join(dst, "ncu_traffic.json")
    traffic = json.load(open(traffic_path)) if os.path.exists(traffic_path) else {}
    for cap, point in CAPTURES.items():
        raw = os.path.join(src, f"{cap}.raw.csv")
        if not os.path.exists(raw):
            continue
        s = ncu_raw_summary.summary(raw)[0]
        with open(os.path.join(dst, f"{tag}_ncu_{cap}.txt"), "w") as fh:
            fh.write(f"# ncu --set full --clock-control none, {point}\n")
            for k, v in s.items():
                fh.write(f"{k}: {v}\n")
        traffic[point] = round(dram_bytes(s["dram__bytes_read.sum"]) + dram_bytes(s["dram__bytes_write.sum"]))
    json.dump(traffic, open(traffic_path, "w"), indent=1)
    print("profiles written:", sorted(os.listdir(dst)))


if __name__ == "__main__":
    main()
