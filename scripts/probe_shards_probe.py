import json, statistics, sys, os
sys.path.insert(0, os.getcwd())
import torch, dockgen as g
import paper_conf_ipps_sukhwanih10_b200 as D
c = g.CONFIGS['prod']; dev = torch.device('cuda', 0)
R, w = g.receptor_ftmap_like(c.n, c.P), g.weights(c.P)
pl = g.probes(c.n_probes, c.m, c.P)
probes = [{"xyz": torch.from_numpy(p.xyz).to(dev), "coef": torch.from_numpy(p.coef).to(dev), "m": p.m} for p in pl]
rot = torch.from_numpy(g.rotations(c.n_rot)).to(dev)
ctx = D.dock_init(torch.from_numpy(R).to(dev), torch.from_numpy(w).to(dev), g.SPACING, m_max=c.m, device=0)
flush = torch.empty(64 << 20, dtype=torch.float32, device=dev)
def t(ps, rs):
    ps2 = D.dock_probes(ctx, ps); units = len(ps) * rs.shape[0]
    out = torch.empty((units, c.k, 4), dtype=torch.int32, device=dev)
    for _ in range(3): D.dock_probe_batch(ctx, ps2, rs, 0, units, c.k, 1, out=out)
    D.dock_sync(ctx); ts = []
    for i in range(8):
        flush.fill_(float(i)); e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(); D.dock_probe_batch(ctx, ps2, rs, 0, units, c.k, 1, out=out); e1.record(); e1.synchronize(); ts.append(e0.elapsed_time(e1))
    D.dock_sync(ctx); info = D.dock_get_info(ctx)
    return round(statistics.median(ts), 3), round(info['corr_ms_last'], 3), info['tc_ksteps_exec_last']
res = {}
res['probe_pairs'] = [(i, pl[2*i].n_atoms, pl[2*i+1].n_atoms, t(probes[2*i:2*i+2], rot)) for i in range(8)]
order = sorted(range(16), key=lambda i: -pl[i].n_atoms)
pairs = [(order[i], order[15 - i]) for i in range(8)]
res['balanced_pairs'] = [(a, b, pl[a].n_atoms, pl[b].n_atoms, t([probes[a], probes[b]], rot)) for a, b in pairs]
res['rot_shard0'] = t(probes, rot[0:62])
res['full'] = t(probes, rot)
print(json.dumps(res))
