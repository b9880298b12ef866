#!/usr/bin/env python
"""Per-rank shard times of the multi-GPU rotation sharding, measured on ONE B200 (this sandbox has one GPU per
call): for N in 1, 2, 4, 8 the unit block rank 0 would own (parallel.shard_range) is docked alone, steps
enqueued back to back (the asynchronous path), CUDA-event timed.  The N-GPU step would add one NCCL
all-gather of N x 16 B x k x units/N poses (64 KB per rank at N = 8); it is NOT included.  The output is a
projection input (per-rank work), not a multi-GPU measurement.   python scripts/shard_times.py [--config prod]"""
import argparse
import json
import os
import statistics
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import dockgen as g  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="prod")
    ap.add_argument("--rotations", type=int, default=0)
    ap.add_argument("--steps", type=int, default=10)
    args = ap.parse_args()
    import dataclasses
    import torch
    import paper_conf_ipps_sukhwanih10_b200 as D
    from paper_conf_ipps_sukhwanih10_b200 import parallel
    c = g.CONFIGS[args.config]
    if args.rotations:
        c = dataclasses.replace(c, n_rot=args.rotations)
    dev = torch.device("cuda", 0)
    R, w = g.receptor_ftmap_like(c.n, c.P), g.weights(c.P)
    probes = [{"xyz": torch.from_numpy(p.xyz).to(dev), "coef": torch.from_numpy(p.coef).to(dev), "m": p.m}
              for p in g.probes(c.n_probes, c.m, c.P)]
    rot = torch.from_numpy(g.rotations(c.n_rot)).to(dev)
    ctx = D.dock_init(torch.from_numpy(R).to(dev), torch.from_numpy(w).to(dev), g.SPACING, m_max=c.m, device=0)
    probes = D.dock_probes(ctx, probes)   # descriptors marshalled once, as bench.py does
    n = c.n_probes * c.n_rot
    flush = torch.empty(64 << 20, dtype=torch.float32, device=dev)
    res = {"config": args.config, "units": n, "note": __doc__.split("\n")[1].strip(), "per_n": {}}
    for N in (1, 2, 4, 8):
        b, e = parallel.shard_range(n, 0, N)
        out = torch.empty((e - b, c.k, 4), dtype=torch.int32, device=dev)
        for _ in range(3):
            D.dock_probe_batch(ctx, probes, rot, b, e, c.k, 1, out=out)
        D.dock_sync(ctx)
        ts = []
        for i in range(args.steps):
            flush.fill_(float(i))
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            D.dock_probe_batch(ctx, probes, rot, b, e, c.k, 1, out=out)
            e1.record()
            e1.synchronize()
            ts.append(e0.elapsed_time(e1))
        D.dock_sync(ctx)
        info = D.dock_get_info(ctx)
        res["per_n"][N] = {"units_rank0": e - b, "ms_median": statistics.median(ts), "ms_min": min(ts),
                           "engine": info["engine_last"], "kernel_ms": info["corr_ms_last"]}
    t1 = res["per_n"][1]["ms_median"]
    for N, r in res["per_n"].items():
        r["projected_efficiency_without_allgather"] = t1 / (N * r["ms_median"])
    print(json.dumps(res), flush=True)
    ctx.close()


if __name__ == "__main__":
    main()
