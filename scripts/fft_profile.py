"""One FFT-engine dock_probe_batch (128^3, P = 4, m = 4, 64 rotations) for an ncu launch list."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import dockgen as g  # noqa: E402
import paper_conf_ipps_sukhwanih10_b200 as D  # noqa: E402

R = g.receptor_ftmap_like((128, 128, 128), 4)
ctx = D.dock_init(R, g.weights(4), g.SPACING, m_max=4)
D.dock_set_tuning(ctx, D.DOCK_TUNE_ENGINE, 3)
probes, rot = g.probes(1, 4, 4), g.rotations(64)
for _ in range(2):
    D.dock_probe_batch(ctx, probes, rot, k=4, rho=1)
ctx.close()
