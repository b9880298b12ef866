"""ctypes declarations of include/dock.h (argument marshalling only).

The library is loaded from this package directory.  There is no fallback: if
libdock.so is missing the import fails loudly (build it with
``python -m paper_conf_ipps_sukhwanih10_b200.build`` or ``__graft_entry__.build()``).
"""
from __future__ import annotations

import ctypes as C
import os

_PKG = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_PKG, "libdock.so")

DOCK_OK = 0
DOCK_MAX_TERMS = 32
DOCK_MAX_M = 8
DOCK_MAX_K = 32
DOCK_POSE_FALLBACK = 1
DOCK_POSE_EMPTY = 2
DOCK_TUNE_REGIONS = 1
DOCK_TUNE_FORCE_FALLBACK = 2
DOCK_TUNE_CAND_CAP = 3
DOCK_TUNE_ENGINE = 4
DOCK_TUNE_TC_VARIANT = 5
DOCK_TUNE_TC_EPILOGUE_WARPS = 6
DOCK_TUNE_TC_CHUNK = 7
DOCK_TUNE_TC_SCHEDULE = 8
DOCK_TUNE_SHARD = 9
DOCK_ENGINE_AUTO, DOCK_ENGINE_FFMA, DOCK_ENGINE_TC, DOCK_ENGINE_FFT, DOCK_ENGINE_SPARSE = 0, 1, 2, 3, 4

STATUS_NAMES = {0: "DOCK_OK", -1: "DOCK_E_INVALID_ARG", -2: "DOCK_E_UNSUPPORTED",
                -3: "DOCK_E_PROBE_OUTSIDE_GRID", -4: "DOCK_E_BAD_ROTATION", -5: "DOCK_E_CUDA",
                -6: "DOCK_E_OOM"}


class dock_pose(C.Structure):
    _fields_ = [("rot", C.c_int32), ("t_lin", C.c_int32), ("score", C.c_float), ("flags", C.c_uint32)]


class dock_grid_desc(C.Structure):
    _fields_ = [("nx", C.c_int), ("ny", C.c_int), ("nz", C.c_int), ("n_terms", C.c_int), ("m_max", C.c_int),
                ("device", C.c_int), ("spacing", C.c_double), ("stream", C.c_void_p)]


class dock_probe_desc(C.Structure):
    _fields_ = [("n_atoms", C.c_int), ("m", C.c_int), ("xyz", C.c_void_p), ("coef", C.c_void_p)]


class dock_info(C.Structure):
    _fields_ = [("lanes_x", C.c_int), ("tile_x", C.c_int), ("tile_y", C.c_int), ("tile_z", C.c_int),
                ("n_tiles", C.c_int), ("n_stages", C.c_int), ("smem_bytes", C.c_int),
                ("regions_last", C.c_int), ("items_last", C.c_int64), ("fallback_last", C.c_int64),
                ("cand_max_last", C.c_int64), ("kernels_last", C.c_int64), ("rot_batch", C.c_int),
                ("x_per_thread", C.c_int), ("padded_x", C.c_int), ("padded_y", C.c_int),
                ("padded_z", C.c_int), ("l2_bytes", C.c_double), ("corr_ms_last", C.c_double),
                ("n_sms", C.c_int), ("engine_last", C.c_int), ("tc_available", C.c_int),
                ("tc_variant_last", C.c_int), ("tc_ksteps_last", C.c_int),
                ("tc_row_last", C.c_int), ("tc_rows_per_tile_last", C.c_int), ("pending", C.c_int),
                ("fb_chunk", C.c_int), ("sp_atom_grids_last", C.c_int), ("sp_row_last", C.c_int),
                ("sp_terms_last", C.c_double), ("sp_zt_last", C.c_int),
                ("tc_ksteps_exec_last", C.c_double)]


EXPORTS = ["dock_init", "dock_probe", "dock_probe_batch", "dock_sync", "dock_score_grid", "dock_voxelize",
           "dock_set_tuning", "dock_get_info", "dock_destroy", "dock_status_string", "dock_last_error",
           "dock_em_init", "dock_em_eval", "dock_em_last_ms", "dock_em_destroy", "dock_em_last_error"]


class dock_em_desc(C.Structure):
    _fields_ = [("n_atoms", C.c_int), ("n_pairs", C.c_int), ("n_types", C.c_int), ("device", C.c_int),
                ("eps_s", C.c_double), ("rc", C.c_double), ("stream", C.c_void_p)]


class dock_em_params(C.Structure):
    _fields_ = [("q", C.c_void_p), ("R", C.c_void_p), ("V", C.c_void_p), ("eps", C.c_void_p), ("rm", C.c_void_p),
                ("type", C.c_void_p), ("omega", C.c_void_p), ("sigma", C.c_void_p), ("mu", C.c_void_p),
                ("pairs", C.c_void_p)]

_lib = None


def lib() -> C.CDLL:
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(LIB_PATH):
        raise ImportError(f"libdock.so not built at {LIB_PATH}; run __graft_entry__.build() "
                          "(the CUDA path has no CPU fallback)")
    L = C.CDLL(LIB_PATH)
    vp, i, i64 = C.c_void_p, C.c_int, C.c_int64
    L.dock_init.argtypes = [C.POINTER(dock_grid_desc), vp, vp, C.POINTER(vp)]
    L.dock_probe.argtypes = [vp, C.POINTER(dock_probe_desc), vp, i, i, i, vp]
    L.dock_probe_batch.argtypes = [vp, C.POINTER(dock_probe_desc), i, vp, i, i64, i64, i, i, vp]
    L.dock_sync.argtypes = [vp]
    L.dock_score_grid.argtypes = [vp, C.POINTER(dock_probe_desc), vp, vp, vp]
    L.dock_voxelize.argtypes = [vp, C.POINTER(dock_probe_desc), vp, i, vp]
    L.dock_set_tuning.argtypes = [vp, i, i64]
    L.dock_get_info.argtypes = [vp, C.POINTER(dock_info)]
    L.dock_destroy.argtypes = [vp]
    L.dock_destroy.restype = None
    L.dock_status_string.argtypes = [i]
    L.dock_status_string.restype = C.c_char_p
    L.dock_last_error.argtypes = [vp]
    L.dock_last_error.restype = C.c_char_p
    L.dock_em_init.argtypes = [C.POINTER(dock_em_desc), C.POINTER(dock_em_params), C.POINTER(vp)]
    L.dock_em_eval.argtypes = [vp, vp, i, vp, vp]
    L.dock_em_last_ms.argtypes = [vp]
    L.dock_em_last_ms.restype = C.c_double
    L.dock_em_destroy.argtypes = [vp]
    L.dock_em_destroy.restype = None
    L.dock_em_last_error.argtypes = [vp]
    L.dock_em_last_error.restype = C.c_char_p
    L.dock_em_init.restype = C.c_int
    L.dock_em_eval.restype = C.c_int
    for name in ("dock_init", "dock_probe", "dock_probe_batch", "dock_sync", "dock_score_grid", "dock_voxelize",
                 "dock_set_tuning", "dock_get_info"):
        getattr(L, name).restype = C.c_int
    _lib = L
    return L
