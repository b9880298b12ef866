"""Binding of the energy-minimisation non-bonded kernels (include/dock_em.h): argument
marshalling only, every step runs in libdock.so's CUDA kernels."""
from __future__ import annotations

import ctypes as C

import numpy as np

from . import _native as N
from .dock import DockError, _buf, _is_torch, _torch


class EmContext:
    def __init__(self, ptr: int, n_atoms: int, device: int):
        self.ptr = C.c_void_p(ptr)
        self.n_atoms, self.device = n_atoms, device

    def close(self):
        if self.ptr:
            N.lib().dock_em_destroy(self.ptr)
            self.ptr = C.c_void_p(0)

    def __del__(self):  # pragma: no cover
        try:
            self.close()
        except Exception:
            pass


def _check(ptr, st):
    if st != N.DOCK_OK:
        msg = N.lib().dock_em_last_error(ptr) if ptr else b""
        raise DockError(st, (msg or b"").decode(errors="replace"))


def em_init(system, device: int | None = None, stream=None) -> EmContext:
    """Copy a system (an object with q, R, V, eps, rm, type, omega, sigma, mu, pairs, eps_s, rc -- e.g.
    dockgen.EmSystem) to the device and build its forward/reverse pair segments."""
    torch = _torch()
    device = torch.cuda.current_device() if device is None else device
    sh = torch.cuda.current_stream(device).cuda_stream if stream is None else (
        stream if isinstance(stream, int) else stream.cuda_stream)
    if sh == 0:
        sh = 1   # cudaStreamLegacy: torch's default stream
    keep = []

    def ptr(x, dt):
        p, k = _buf(x, dt)
        keep.append(k)
        return C.c_void_p(p)

    pairs = np.ascontiguousarray(system.pairs, dtype=np.int32).reshape(-1, 2)
    T = int(np.asarray(system.omega).shape[0])
    d = N.dock_em_desc(int(np.asarray(system.q).shape[0]), int(pairs.shape[0]), T, device, float(system.eps_s),
                       float(system.rc), C.c_void_p(sh))
    p = N.dock_em_params(ptr(system.q, "f8"), ptr(system.R, "f8"), ptr(system.V, "f8"), ptr(system.eps, "f8"),
                         ptr(system.rm, "f8"), ptr(system.type, "i4"), ptr(system.omega, "f8"),
                         ptr(system.sigma, "f8"), ptr(system.mu, "f8"), ptr(pairs, "i4"))
    out = C.c_void_p()
    with torch.cuda.device(device):
        st = N.lib().dock_em_init(C.byref(d), C.byref(p), C.byref(out))
    _check(None, st)
    return EmContext(out.value, d.n_atoms, device)


def em_eval(ctx: EmContext, x, forces: bool = True):
    """x [n_conf][n_atoms][3] float64 (numpy, or a torch tensor on the context's device) ->
    (E [n_conf][3] = (E_self, E_GB, E_vdw), F [n_conf][n_atoms][3] or None) as numpy arrays."""
    torch = _torch()
    if _is_torch(x) and x.is_cuda and x.device.index != ctx.device:
        raise ValueError("coordinates on another device")
    xp, xk = _buf(x, "f8")
    if tuple(xk.shape[-2:]) != (ctx.n_atoms, 3):
        raise ValueError(f"coordinates must be [n_conf][{ctx.n_atoms}][3]")
    nc = 1 if xk.ndim == 2 else int(xk.shape[0])
    e = np.zeros((nc, 3))
    f = np.zeros((nc, ctx.n_atoms, 3)) if forces else None
    with torch.cuda.device(ctx.device):
        st = N.lib().dock_em_eval(ctx.ptr, C.c_void_p(xp), nc, C.c_void_p(e.ctypes.data),
                                  C.c_void_p(f.ctypes.data) if forces else None)
    _check(ctx.ptr, st)
    return e, f


def em_last_ms(ctx: EmContext) -> float:
    return float(N.lib().dock_em_last_ms(ctx.ptr))
