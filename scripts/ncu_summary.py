#!/usr/bin/env python
"""Summarise an ncu capture brought back by scripts/ncu_kernel.sh: speed-of-light, scheduler and the top
stall reasons, plus the hottest SASS lines.  usage: ncu_summary.py TAG"""
import csv
import gzip
import sys

tag = sys.argv[1]
rows = list(csv.reader(open(f"gpurun_out/ncu_{tag}_details.csv")))
h = rows[0]
keep = ("GPU Speed Of Light Throughput", "Compute Workload Analysis", "Scheduler Statistics", "Occupancy",
        "Memory Workload Analysis", "Warp State Statistics")
for r in rows[1:]:
    d = dict(zip(h, r))
    if d.get("Section Name") in keep and d["Metric Name"] in (
            "Duration", "Compute (SM) Throughput", "Memory Throughput", "L1/TEX Cache Throughput",
            "L2 Cache Throughput", "DRAM Throughput", "Executed Ipc Active", "Issue Slots Busy",
            "Eligible Warps Per Scheduler", "Active Warps Per Scheduler", "Achieved Occupancy",
            "Warp Cycles Per Issued Instruction", "L2 Hit Rate", "Mem Pipes Busy"):
        print(f"{d['Metric Name']:36s} {d['Metric Value']} {d.get('Metric Unit', '')}")
rows = list(csv.reader(gzip.open(f"gpurun_out/ncu_{tag}_source.csv.gz", "rt")))
h = rows[1]
data = rows[2:]
iS = h.index("Warp Stall Sampling (All Samples)")
iE = h.index("Instructions Executed")
iSrc = h.index("Source")
sc = [i for i, c in enumerate(h) if c.startswith("stall_") and "Not Issued" not in c]
agg = {}
for r in data:
    for i in sc:
        agg[h[i]] = agg.get(h[i], 0) + int(r[i] or 0)
tot = sum(agg.values())
print("stalls:", ", ".join(f"{k[6:]} {v / tot:.0%}" for k, v in sorted(agg.items(), key=lambda x: -x[1])[:8]))
print("instructions executed:", sum(int(r[iE]) for r in data))
for r in sorted(data, key=lambda r: -int(r[iS]))[:int(sys.argv[2]) if len(sys.argv) > 2 else 20]:
    st = max(sc, key=lambda i: int(r[i] or 0))
    print(f"{r[0][-5:]} {r[iSrc][:60]:60s} samples {r[iS]:>6} exec {r[iE]:>9} {h[st][6:]}")
