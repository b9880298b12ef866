"""Probe (not product code): scheduler chunk size for one block-sharded rank (N = 8, rank 0) at prod."""
import os, sys, statistics
sys.path.insert(0, os.getcwd())
import torch, dockgen as g
import paper_conf_ipps_sukhwanih10_b200 as D
c = g.CONFIGS["prod"]; dev = torch.device("cuda", 0)
R, w = g.receptor_ftmap_like(c.n, c.P), g.weights(c.P)
probes = D.dock_probes(None, []) if False else None
ctx = D.dock_init(torch.from_numpy(R).to(dev), torch.from_numpy(w).to(dev), g.SPACING, m_max=c.m, device=0)
probes = D.dock_probes(ctx, [{"xyz": torch.from_numpy(p.xyz).to(dev), "coef": torch.from_numpy(p.coef).to(dev), "m": p.m}
                             for p in g.probes(c.n_probes, c.m, c.P)])
rot = torch.from_numpy(g.rotations(c.n_rot)).to(dev)
n = c.n_probes * c.n_rot
out = torch.full((n, c.k, 4), -2 ** 31, dtype=torch.int32, device=dev)
D.dock_set_tuning(ctx, D.DOCK_TUNE_SHARD, (8 << 16) | 0)
for chunk in (1, 2, 3, 4, 6):
    D.dock_set_tuning(ctx, D.DOCK_TUNE_TC_CHUNK, chunk)
    ks = []
    for i in range(8):
        D.dock_probe_batch(ctx, probes, rot, 0, n, c.k, 1, out=out)
        D.dock_sync(ctx)
        ks.append(D.dock_get_info(ctx)["corr_ms_last"])
    print("chunk", chunk, "kernel ms median", round(statistics.median(ks[2:]), 4), flush=True)
