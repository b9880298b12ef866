"""Probe (not product code): DOCK_TC_TRACE counters of one block-sharded rank (N = 8, rank 0) against the full
prod launch, to see why a rank's kernel costs more per tile than 1/N of the full one."""
import os, sys
sys.path.insert(0, os.getcwd())
os.environ["DOCK_TC_TRACE"] = "1"
import torch, dockgen as g
import paper_conf_ipps_sukhwanih10_b200 as D
c = g.CONFIGS["prod"]; dev = torch.device("cuda", 0)
R, w = g.receptor_ftmap_like(c.n, c.P), g.weights(c.P)
probes = [{"xyz": torch.from_numpy(p.xyz).to(dev), "coef": torch.from_numpy(p.coef).to(dev), "m": p.m}
          for p in g.probes(c.n_probes, c.m, c.P)]
rot = torch.from_numpy(g.rotations(c.n_rot)).to(dev)
ctx = D.dock_init(torch.from_numpy(R).to(dev), torch.from_numpy(w).to(dev), g.SPACING, m_max=c.m, device=0)
n = c.n_probes * c.n_rot
out = torch.full((n, c.k, 4), -2 ** 31, dtype=torch.int32, device=dev)
for world, rank in ((1, 0), (8, 0), (8, 3)):
    D.dock_set_tuning(ctx, D.DOCK_TUNE_SHARD, (world << 16) | rank)
    for _ in range(2):
        D.dock_probe_batch(ctx, probes, rot, 0, n, c.k, 1, out=out)
    D.dock_sync(ctx)
    print("world", world, "rank", rank, "kernel ms", D.dock_get_info(ctx)["corr_ms_last"], flush=True)
