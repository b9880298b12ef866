"""ctypes marshalling for oracle/dock_oracle.c (TEST INFRASTRUCTURE ONLY; see __init__)."""
from __future__ import annotations

import ctypes as C
import os
import subprocess
import threading
from typing import Sequence, Tuple

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "dock_oracle.c")
_LIB_PATH = os.path.join(_HERE, "liboracle.so")
_lib = None
_lock = threading.Lock()


class OracleError(RuntimeError):
    pass


def build_oracle(force: bool = False) -> str:
    """Compile dock_oracle.c -> liboracle.so (gcc -O2 -fopenmp; no -ffast-math)."""
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < os.path.getmtime(_SRC):
        tmp = _LIB_PATH + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O2", "-fopenmp", "-fPIC", "-shared", "-std=c99",
                               "-o", tmp, _SRC, "-lm"])
        os.replace(tmp, _LIB_PATH)
    return _LIB_PATH


def _L():
    global _lib
    with _lock:
        if _lib is None:
            build_oracle()
            lib = C.CDLL(_LIB_PATH)
            dp, fp, ip, lp = (C.POINTER(C.c_double), C.POINTER(C.c_float), C.POINTER(C.c_int),
                              C.POINTER(C.c_int64))
            lib.orc_check_rotation.argtypes = [dp]
            lib.orc_voxelize.argtypes = [dp, fp, C.c_int, C.c_int, C.c_int, dp, C.c_double, dp]
            lib.orc_score_grid.argtypes = [fp, C.c_int, C.c_int, C.c_int, C.c_int, dp, C.c_int, fp, dp, dp]
            lib.orc_score_grid.restype = None
            lib.orc_filter.argtypes = [dp, C.c_int, C.c_int, C.c_int, C.c_int, C.c_int, lp, dp]
            lib.orc_dock.argtypes = [fp, C.c_int, C.c_int, C.c_int, C.c_int, fp, C.c_double,
                                     dp, fp, ip, ip, C.c_int, dp, C.c_int, C.c_int64, C.c_int64,
                                     C.c_int, C.c_int, C.c_int, lp, dp, dp, ip]
            lib.orc_max_threads.argtypes = []
            _lib = lib
    return _lib


def _p(a: np.ndarray, ct):
    return a.ctypes.data_as(C.POINTER(ct))


def _f32(a):
    return np.ascontiguousarray(a, dtype=np.float32)


def _f64(a):
    return np.ascontiguousarray(a, dtype=np.float64)


def max_threads() -> int:
    return int(_L().orc_max_threads())


def check_rotation(q: np.ndarray) -> int:
    return int(_L().orc_check_rotation(_p(_f64(q).reshape(9), C.c_double)))


def voxelize(xyz: np.ndarray, coef: np.ndarray, m: int, rot9: np.ndarray, spacing: float) -> np.ndarray:
    """Rotated, voxelized probe grids L ``[P][m][m][m]`` float64."""
    xyz, coef = _f64(xyz).reshape(-1, 3), _f32(coef)
    n = xyz.shape[0]
    P = coef.shape[1] if coef.ndim == 2 else 1
    L = np.zeros((P, m, m, m), dtype=np.float64)
    st = _L().orc_voxelize(_p(xyz, C.c_double), _p(coef, C.c_float), n, P, m,
                           _p(_f64(rot9).reshape(9), C.c_double), float(spacing), _p(L, C.c_double))
    if st != 0:
        raise OracleError(f"voxelize status {st}")
    return L


def score_grid(R: np.ndarray, L: np.ndarray, w: np.ndarray, with_A: bool = True):
    """S (and A) ``[nz][ny][nx]`` float64 per Eq. 1/2."""
    R, L, w = _f32(R), _f64(L), _f32(w)
    P, nz, ny, nx = R.shape
    m = L.shape[-1]
    assert L.shape == (P, m, m, m) and w.shape == (P,)
    S = np.empty((nz, ny, nx), dtype=np.float64)
    A = np.empty_like(S) if with_A else None
    _L().orc_score_grid(_p(R, C.c_float), nx, ny, nz, P, _p(L, C.c_double), m, _p(w, C.c_float),
                        _p(S, C.c_double), _p(A, C.c_double) if with_A else None)
    return (S, A) if with_A else S


def filter_greedy(S: np.ndarray, k: int, rho: int) -> Tuple[np.ndarray, np.ndarray]:
    """Greedy best-then-exclude filter: (t_lin[k'], score[k'])."""
    S = _f64(S)
    nz, ny, nx = S.shape
    t = np.full(k, -1, dtype=np.int64); s = np.full(k, np.nan)
    n = _L().orc_filter(_p(S, C.c_double), nx, ny, nz, k, rho, _p(t, C.c_int64), _p(s, C.c_double))
    if n < 0:
        raise OracleError("filter failed")
    return t[:n], s[:n]


def dock(R: np.ndarray, w: np.ndarray, spacing: float, probes, rot: np.ndarray, k: int, rho: int,
         unit_begin: int = 0, unit_end: int | None = None, n_threads: int = 0, with_A: bool = False):
    """Full docking over probe-major (probe, rotation) units -> (t_lin [U][k], score [U][k], status [U]),
    and with ``with_A`` also the magnitude sum A [U][k] at each pick (reading Q16)."""
    R, w, rot = _f32(R), _f32(w), _f64(rot).reshape(-1, 9)
    P, nz, ny, nx = R.shape
    n_rot = rot.shape[0]
    if unit_end is None:
        unit_end = len(probes) * n_rot
    xyz = _f64(np.concatenate([p.xyz.reshape(-1, 3) for p in probes], axis=0)) if probes else np.zeros((0, 3))
    coef = _f32(np.concatenate([p.coef.reshape(-1, P) for p in probes], axis=0)) if probes else np.zeros((0, P))
    off = np.zeros(len(probes) + 1, dtype=np.int32)
    off[1:] = np.cumsum([p.xyz.shape[0] for p in probes])
    ms = np.ascontiguousarray([p.m for p in probes], dtype=np.int32)
    U = unit_end - unit_begin
    out_t = np.full((U, k), -1, dtype=np.int64)
    out_s = np.full((U, k), np.nan)
    out_a = np.full((U, k), np.nan) if with_A else None
    st = np.zeros(U, dtype=np.int32)
    rc = _L().orc_dock(_p(R, C.c_float), nx, ny, nz, P, _p(w, C.c_float), float(spacing),
                       _p(xyz, C.c_double), _p(coef, C.c_float), _p(off, C.c_int), _p(ms, C.c_int),
                       len(probes), _p(rot, C.c_double), n_rot, unit_begin, unit_end, k, rho, n_threads,
                       _p(out_t, C.c_int64), _p(out_s, C.c_double),
                       _p(out_a, C.c_double) if with_A else None, _p(st, C.c_int))
    if rc != 0:
        raise OracleError(f"dock status {rc}")
    return (out_t, out_s, st, out_a) if with_A else (out_t, out_s, st)
