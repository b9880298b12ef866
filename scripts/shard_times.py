#!/usr/bin/env python
"""Per-rank shard times of the multi-GPU rotation sharding, measured on ONE B200 (this sandbox has one GPU per
call): for N in 1, 2, 4, 8 every rank's shard is docked alone, CUDA-event timed, and the projection takes the
slowest rank.  Two shardings: "rotations" (every probe over the rank's rotation slice, parallel.dock_probe_sharded)
and "blocks" (DOCK_TUNE_SHARD: every rank clusters all units and docks its blocks of the common block order,
parallel.dock_probe_sharded_blocks; the collective is then one all-reduce MAX).  The N-GPU step would add one NCCL
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
    res = {"config": args.config, "units": n, "note": "per-rank shard times on one B200 (see the docstring)"}
    def timed(call):
        for _ in range(3):
            call()
        D.dock_sync(ctx)
        ts = []
        for i in range(args.steps):
            flush.fill_(float(i))
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            call()
            e1.record()
            e1.synchronize()
            ts.append(e0.elapsed_time(e1))
        D.dock_sync(ctx)
        info = D.dock_get_info(ctx)
        return statistics.median(ts), info["corr_ms_last"], info["engine_last"]

    full = torch.empty((n, c.k, 4), dtype=torch.int32, device=dev)
    for mode in ("rotations", "blocks"):
        res[mode] = {}
        for N in (1, 2, 4, 8):
            ranks = []
            for rk in range(N):
                if mode == "rotations":   # every probe over this rank's rotation slice
                    r0, r1 = parallel.shard_range(c.n_rot, rk, N)
                    units = c.n_probes * (r1 - r0)
                    out = torch.empty((units, c.k, 4), dtype=torch.int32, device=dev)
                    rs = rot[r0:r1]
                    ms, kms, eng = timed(lambda: D.dock_probe_batch(ctx, probes, rs, 0, units, c.k, 1, out=out))
                    ranks.append({"rotations": [r0, r1], "units": units, "ms_median": ms, "kernel_ms": kms,
                                  "engine": eng})
                else:   # DOCK_TUNE_SHARD: all units clustered, this rank's blocks docked
                    D.dock_set_tuning(ctx, D.DOCK_TUNE_SHARD, (N << 16) | rk)
                    try:
                        ms, kms, eng = timed(lambda: D.dock_probe_batch(ctx, probes, rot, 0, n, c.k, 1, out=full))
                    except D.DockError as ex:
                        ranks = None
                        res[mode]["unsupported"] = str(ex)
                        break
                    finally:
                        D.dock_set_tuning(ctx, D.DOCK_TUNE_SHARD, 1 << 16)
                    ranks.append({"rank": rk, "ms_median": ms, "kernel_ms": kms, "engine": eng})
            if ranks is None:
                break
            res[mode][N] = {"ranks": ranks, "ms_max_over_ranks": max(r["ms_median"] for r in ranks),
                            "ms_mean_over_ranks": statistics.mean(r["ms_median"] for r in ranks)}
        if 1 in res[mode]:
            t1 = res[mode][1]["ms_max_over_ranks"]
            for N, r in res[mode].items():
                if isinstance(r, dict):
                    r["projected_efficiency_without_collective"] = t1 / (N * r["ms_max_over_ranks"])
    print(json.dumps(res), flush=True)
    ctx.close()


if __name__ == "__main__":
    main()
