#!/usr/bin/env python
"""Host gaps inside the asynchronous docking step, measured with CUPTI
through torch.profiler (nsys is not installed): the device timeline of every kernel and copy of K steps
of the bench workload enqueued back to back, and the largest idle gap between consecutive device
activities inside a step.  python scripts/host_gaps.py [--config prod] [--steps 5]"""
import argparse
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import dockgen as g  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="prod")
    ap.add_argument("--steps", type=int, default=8)
    ap.add_argument("--engine", default="auto", choices=["auto", "tc", "sparse", "ffma"])
    args = ap.parse_args()
    import torch
    from torch.profiler import ProfilerActivity, profile
    import paper_conf_ipps_sukhwanih10_b200 as D
    c = g.CONFIGS[args.config]
    dev = torch.device("cuda", 0)
    R, w = g.receptor_ftmap_like(c.n, c.P), g.weights(c.P)
    probes = [{"xyz": torch.from_numpy(p.xyz).to(dev), "coef": torch.from_numpy(p.coef).to(dev), "m": p.m}
              for p in g.probes(c.n_probes, c.m, c.P)]
    rot = torch.from_numpy(g.rotations(c.n_rot)).to(dev)
    ctx = D.dock_init(torch.from_numpy(R).to(dev), torch.from_numpy(w).to(dev), g.SPACING, m_max=c.m, device=0)
    probes = D.dock_probes(ctx, probes)   # descriptors marshalled once, as bench.py does
    D.dock_set_tuning(ctx, D.DOCK_TUNE_ENGINE, {"auto": 0, "ffma": 1, "tc": 2, "sparse": 4}[args.engine])
    n = c.n_probes * c.n_rot
    out = torch.empty((n, c.k, 4), dtype=torch.int32, device=dev)
    for _ in range(3):
        D.dock_probe_batch(ctx, probes, rot, 0, n, c.k, 1, out=out)
    D.dock_sync(ctx)
    with profile(activities=[ProfilerActivity.CUDA]) as prof:
        for _ in range(args.steps):
            D.dock_probe_batch(ctx, probes, rot, 0, n, c.k, 1, out=out)   # asynchronous: no host sync
        D.dock_sync(ctx)
    evs = sorted([e for e in prof.events() if e.device_type.name == "CUDA"], key=lambda e: e.time_range.start)
    spans = [(e.time_range.start, e.time_range.end, e.name) for e in evs]
    # steps start at the gather kernel of each call
    starts = [i for i, s in enumerate(spans) if "k_gather_probes" in s[2]]
    gaps, first = [], []   # the first profiled step starts on an idle GPU: its gaps are host enqueue time
    for si, i0 in enumerate(starts):
        i1 = starts[si + 1] if si + 1 < len(starts) else len(spans)
        step = spans[i0:i1]
        end = step[0][1]
        for a, b, nm in step[1:]:
            (first if si == 0 else gaps).append((a - end, nm))
            end = max(end, b)
    inter = [spans[starts[i + 1]][0] - max(b for _, b, _ in spans[starts[i]:starts[i + 1]])
             for i in range(len(starts) - 1)]
    worst = max(gaps) if gaps else (0, "")
    line = {"config": args.config, "engine": D.dock_get_info(ctx)["engine_last"], "steps": args.steps,
            "device_activities": len(spans), "kernels_per_step": len(spans) // max(1, len(starts)),
            "max_gap_inside_step_us": worst[0], "before_kernel": worst[1][:60],
            "max_gap_inside_first_step_us": max(first)[0] if first else None,
            "steps_in_gap_stats": "2.." + str(len(starts)) + " (steady state: the GPU never waits for the host)",
            "median_gap_inside_step_us": sorted(x for x, _ in gaps)[len(gaps) // 2] if gaps else 0,
            "max_gap_between_steps_us": max(inter) if inter else None,
            "timer": "CUPTI activity timestamps (torch.profiler), steps enqueued back to back"}
    print(json.dumps(line), flush=True)
    ctx.close()


if __name__ == "__main__":
    main()
