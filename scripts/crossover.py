"""Direct-vs-FFT crossover (the paper's claim that direct correlation beats FFT for
small ligand grids), measured on one B200.

For each probe grid size m, 128^3 receptor, P = 4 terms, k = 4, rho = 1: time dock_probe_batch over R
rotations with the FP32 FFMA engine, the tcgen05 engine and the FFT engine (cuFFT + exact greedy on the
score grids); print one JSON line per m and a summary line with the crossover points.
Usage (GPU box): python scripts/crossover.py [--rotations 256] [--out gpurun_out/crossover.json]
"""
import argparse
import json
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402
import torch  # noqa: E402

import dockgen as g  # noqa: E402


def timed(D, ctx, probes, rot, reps=3):
    D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)   # warm-up (plans, buffers)
    best = 1e30
    for _ in range(reps):
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
        torch.cuda.synchronize()
        best = min(best, time.perf_counter() - t0)
    return best


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--rotations", type=int, default=256)
    ap.add_argument("--grid", type=int, default=128)
    ap.add_argument("--out", default="")
    a = ap.parse_args()
    from paper_conf_ipps_sukhwanih10_b200 import build
    build.build_native()
    import paper_conf_ipps_sukhwanih10_b200 as D
    n, P = (a.grid,) * 3, 4
    R = g.receptor_ftmap_like(n, P)
    w = g.weights(P)
    rot = g.rotations(a.rotations)
    ctx = D.dock_init(R, w, g.SPACING, m_max=8)
    rows = []
    for m in range(2, 9):
        probes = g.probes(1, m, P)
        row = {"m": m, "grid": list(n), "P": P, "rotations": a.rotations}
        for name, eng in (("ffma", 1), ("tcgen05", 2), ("fft", 3)):
            D.dock_set_tuning(ctx, D.DOCK_TUNE_ENGINE, eng)
            dt = timed(D, ctx, probes, rot)
            row[name + "_us_per_rot"] = dt / a.rotations * 1e6
            row[name + "_rot_per_s"] = a.rotations / dt
        row["dense_gflop_per_rot"] = 2.0 * P * m ** 3 * np.prod(n) / 1e9
        rows.append(row)
        print(json.dumps(row), flush=True)
    ctx.close()
    cross = {}
    for eng in ("ffma", "tcgen05"):
        faster = [r["m"] for r in rows if r["fft_us_per_rot"] < r[eng + "_us_per_rot"]]
        cross[eng] = min(faster) if faster else None
    summary = {"crossover_m_fft_beats": cross, "rows": rows}
    print(json.dumps({"crossover_m_fft_beats": cross}))
    if a.out:
        with open(a.out, "w") as f:
            json.dump(summary, f, indent=1)


if __name__ == "__main__":
    main()
