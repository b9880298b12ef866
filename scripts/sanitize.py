"""Small docking run for compute-sanitizer (memcheck / racecheck / synccheck): toy-sized receptor, every
engine (FFMA, tcgen05 variant 1, tcgen05 variant 2, FFT, sparse ligand), k = 4, rho = 1, one forced pass
through the device-driven fallback graph per direct engine, an asynchronous device-output call, and the
energy-minimisation kernels.  Run on the GPU box as
  compute-sanitizer --tool memcheck python scripts/sanitize.py
"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import dockgen as g  # noqa: E402
import paper_conf_ipps_sukhwanih10_b200 as D  # noqa: E402

P, m = 4, 4
R = g.receptor_ftmap_like((64, 20, 12), P)
w = g.weights(P)
probes = g.probes(2, m, P)
rot = g.rotations(130)
ctx = D.dock_init(R, w, g.SPACING, m_max=m)
ref = None
for eng, var in ((1, 0), (2, 1), (2, 2), (3, 0), (4, 0)):
    D.dock_set_tuning(ctx, D.DOCK_TUNE_ENGINE, eng)
    D.dock_set_tuning(ctx, D.DOCK_TUNE_TC_VARIANT, var)
    poses = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
    info = D.dock_get_info(ctx)
    same = None if ref is None else float((poses["t_lin"] == ref["t_lin"]).mean())
    ref = poses if ref is None else ref
    print(f"engine {eng} variant {info['tc_variant_last']}: fallback {info['fallback_last']}, t_lin agreement {same}")
    if eng != 3:   # the device-driven exact fallback (CUDA-graph loop), every rotation flagged
        D.dock_set_tuning(ctx, D.DOCK_TUNE_FORCE_FALLBACK, 1)
        fb = D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
        D.dock_set_tuning(ctx, D.DOCK_TUNE_FORCE_FALLBACK, 0)
        print(f"  forced fallback: t_lin agreement {float((fb['t_lin'] == poses['t_lin']).mean())}")
import torch  # noqa: E402
out = torch.empty((len(probes) * len(rot), 4, 4), dtype=torch.int32, device="cuda")
D.dock_probe_batch(ctx, probes, rot, k=4, rho=1, out=out)   # asynchronous device output
D.dock_sync(ctx)
ctx.close()
s = g.em_system(200, seed=3)
ectx = D.em.em_init(s)
e, f = D.em.em_eval(ectx, g.em_conformations(s, 3))
ectx.close()
print("em", e[0])
print("sanitize run done")
