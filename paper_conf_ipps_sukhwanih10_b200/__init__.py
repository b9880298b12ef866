"""B200-native rigid-docking hot path of FTMap (Sukhwani & Herbordt, IPPS 2010).

Public API (same names as the C ABI in include/dock.h):
    dock_init, dock_probe, dock_probe_batch, dock_sync,
    dock_probes (marshal a probe list once: ProbeSet), dock_score_grid, dock_voxelize,
    dock_set_tuning, dock_get_info, dock_destroy
and the multi-GPU shard helper ``parallel.dock_probe_sharded``.
"""
from .dock import (  # noqa: F401
    POSE_DTYPE, DockContext, DockError, ProbeSet, dock_destroy, dock_get_info, dock_init, dock_probe,
    dock_probe_batch, dock_probes, dock_score_grid, dock_set_tuning, dock_sync, dock_voxelize, poses_from_device,
)
from ._native import (  # noqa: F401
    DOCK_MAX_K, DOCK_MAX_M, DOCK_MAX_TERMS, DOCK_POSE_FALLBACK, DOCK_TUNE_CAND_CAP, DOCK_TUNE_ENGINE, DOCK_TUNE_TC_VARIANT, DOCK_TUNE_TC_CHUNK,
    DOCK_TUNE_TC_SCHEDULE, DOCK_TUNE_SHARD,
    DOCK_TUNE_FORCE_FALLBACK, DOCK_TUNE_REGIONS, EXPORTS, LIB_PATH,
)
from . import parallel  # noqa: F401,E402
from . import em  # noqa: F401,E402  (energy-minimisation non-bonded kernels, NEXT-4)
