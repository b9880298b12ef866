import os, sys
sys.path.insert(0, os.getcwd())
import numpy as np, dockgen as g, paper_conf_ipps_sukhwanih10_b200 as D
c = g.CONFIGS["prod"]
R = g.receptor_ftmap_like(c.n, c.P); w = g.weights(c.P)
probes = g.probes(c.n_probes, c.m, c.P); rot = g.rotations(c.n_rot)
ctx = D.dock_init(R, w, g.SPACING, m_max=c.m)
poses = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
info = D.dock_get_info(ctx); print("fallback", info["fallback_last"], "cand_max", info["cand_max_last"])
fl = np.flatnonzero((poses["flags"][:, 0] & 1) != 0)
print("flagged units", fl.tolist())
for u in fl[:5]:
    pr, r = probes[u // 500], u % 500
    S = D.dock_score_grid(ctx, pr, rot[r]).reshape(128, 128, 128)
    t4 = poses[u]["t_lin"][3]; s4 = poses[u]["score"][3]
    better = np.flatnonzero(S.reshape(-1) < s4)
    z, y, x = better // 16384, (better // 128) % 128, better % 128
    print(f"unit {u} probe {u//500} atoms {len(pr.xyz)} picks {poses[u]['t_lin'].tolist()} scores {poses[u]['score'].tolist()}")
    print(f"   cells better than pick4: {better.size}; x range {x.min()}-{x.max()} y {y.min()}-{y.max()} z {z.min()}-{z.max()}")
    # class of a cell for nepi=8 (2 classes): tile row q = y%4, chunk = x//32, class = ((chunk - q) mod 4) % 2
    cls = (((x // 32) - (y % 4)) % 4) % 2
    reg_items = info["regions_last"]
    print("   per-class counts", np.bincount(cls, minlength=2).tolist(), "unique scores among better", np.unique(S.reshape(-1)[better]).size)
ctx.close()
