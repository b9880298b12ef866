"""ctypes marshalling for oracle/em_oracle.c (TEST INFRASTRUCTURE ONLY; see oracle/__init__.py).

The FP64 reference of the non-bonded energy + forces of FTMap's energy minimisation (
PAPER.md Eqs. 4-10, readings E1-E6 in DESIGN.md §13)."""
from __future__ import annotations

import ctypes as C
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "em_oracle.c")
_LIB_PATH = os.path.join(_HERE, "libemoracle.so")
_lib = None
_lock = threading.Lock()


class em_sys(C.Structure):
    _fields_ = [("n_atoms", C.c_int), ("n_pairs", C.c_int), ("n_types", C.c_int),
                ("q", C.c_void_p), ("R", C.c_void_p), ("V", C.c_void_p), ("eps", C.c_void_p), ("rm", C.c_void_p),
                ("type", C.c_void_p), ("omega", C.c_void_p), ("sigma", C.c_void_p), ("mu", C.c_void_p),
                ("pairs", C.c_void_p), ("eps_s", C.c_double), ("rc", C.c_double)]


def build_em_oracle(force: bool = False) -> str:
    if force or not os.path.exists(_LIB_PATH) or os.path.getmtime(_LIB_PATH) < os.path.getmtime(_SRC):
        tmp = _LIB_PATH + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O2", "-fopenmp", "-fPIC", "-shared", "-std=c99", "-o", tmp, _SRC, "-lm"])
        os.replace(tmp, _LIB_PATH)
    return _LIB_PATH


def _L():
    global _lib
    with _lock:
        if _lib is None:
            build_em_oracle()
            lib = C.CDLL(_LIB_PATH)
            lib.orc_em_eval.argtypes = [C.POINTER(em_sys), C.c_void_p, C.c_void_p, C.c_void_p]
            lib.orc_em_eval.restype = None
            lib.orc_em_eval_batch.argtypes = [C.POINTER(em_sys), C.c_int, C.c_void_p, C.c_void_p, C.c_void_p, C.c_int]
            lib.orc_em_eval_batch.restype = None
            _lib = lib
    return _lib


def _sys(s):
    keep = {}

    def arr(name, dt):
        a = np.ascontiguousarray(getattr(s, name), dtype=dt)
        keep[name] = a
        return a.ctypes.data

    st = em_sys(int(s.q.shape[0]), int(s.pairs.shape[0]), int(s.omega.shape[0]),
                arr("q", np.float64), arr("R", np.float64), arr("V", np.float64), arr("eps", np.float64),
                arr("rm", np.float64), arr("type", np.int32), arr("omega", np.float64), arr("sigma", np.float64),
                arr("mu", np.float64), arr("pairs", np.int32), float(s.eps_s), float(s.rc))
    return st, keep


def em_eval(system, x: np.ndarray, forces: bool = True, n_threads: int = 0):
    """x [n_conf][n_atoms][3] (or [n_atoms][3]) -> (E [n_conf][3] = (self, GB, vdW), F [n_conf][n_atoms][3])."""
    x = np.ascontiguousarray(x, dtype=np.float64)
    single = x.ndim == 2
    if single:
        x = x[None]
    nc, n = x.shape[0], x.shape[1]
    e = np.zeros((nc, 3))
    f = np.zeros((nc, n, 3)) if forces else None
    st, keep = _sys(system)
    _L().orc_em_eval_batch(C.byref(st), nc, x.ctypes.data, e.ctypes.data, f.ctypes.data if forces else None,
                           n_threads)
    del keep
    if single:
        return e[0], (f[0] if forces else None)
    return e, f
