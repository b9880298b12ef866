#!/usr/bin/env python
"""Record an ncu --set full capture's DRAM traffic for bench.py's roofline 'traffic' field.

    python scripts/traffic_from_ncu.py gpurun_out/ncu_<tag>_raw.csv CONFIG [--rotations R] [--gpus 1] [--note ...]

Writes profiles/corr_traffic.json["<kernel>@<CONFIG>[@r<R>]"] (the bench launch the capture was taken of) = dram__bytes_read.sum + dram__bytes_write.sum per launch, the
duration and tensor-pipe activity under ncu, and the sha256 of the kernel's SASS in the current
libdock.so; bench.py reports the traffic only while that hash still matches (no stale captures)."""
import argparse
import csv
import json
import os
import re
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import bench  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("raw")
    ap.add_argument("config")
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--rotations", type=int, default=0, help="bench.py --rotations of the captured run")
    ap.add_argument("--note", default="")
    a = ap.parse_args()
    rows = list(csv.reader(open(a.raw)))
    h, units, v = rows[0], rows[1], rows[2]
    d = dict(zip(h, v))
    u = dict(zip(h, units))

    def val(k):
        x = float(d[k].replace(",", ""))
        scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "ms": 1, "us": 1e-3, "ns": 1e-6, "%": 1}
        return x * scale.get(u[k], 1)

    name = d["Kernel Name"]
    m = re.match(r"void (?:\w+::)?(\w+)<(.*)>\(", name)
    args = [t.strip().replace("(int)", "").replace("(bool)", "") for t in m.group(2).split(",")]
    args = ["false" if t == "0" and i == len(args) - 1 else "true" if t == "1" and i == len(args) - 1 else t
            for i, t in enumerate(args)]
    kernel = f"{m.group(1)}<{','.join(args)}>"
    path = os.path.join(ROOT, "profiles", "corr_traffic.json")
    tj = json.load(open(path)) if os.path.exists(path) else {}
    tj["_note"] = ("dram__bytes_read.sum + dram__bytes_write.sum per launch from one ncu --set full capture "
                   "(1 GPU, cold L2 at launch start under ncu); sass_sha256 = the kernel's SASS in libdock.so "
                   "at capture time (bench.py drops the figure when it no longer matches)")
    key = f"{kernel}@{a.config}" + (f"@r{a.rotations}" if a.rotations else "")
    tj[key] = {"config": a.config, "gpus": a.gpus,
                  "dram_bytes_per_launch": val("dram__bytes_read.sum") + val("dram__bytes_write.sum"),
                  "duration_ms_under_ncu": val("gpu__time_duration.sum"),
                  "tensor_pipe_pct": val("sm__pipe_tensor_cycles_active.avg.pct_of_peak_sustained_active"),
                  "source": os.path.basename(a.raw), "sass_sha256": bench.kernel_sass_sha(kernel), "note": a.note}
    json.dump(tj, open(path, "w"), indent=1)
    print(key, tj[key])


if __name__ == "__main__":
    main()
