"""Thin Python binding of the C ABI (include/dock.h), same names as the C entry points.

Argument marshalling only: every step of the hot path (voxelize, correlate, score,
filter) runs in libdock.so's CUDA kernels.  torch is used for device buffers and the
current CUDA stream; numpy arrays are accepted as host buffers.
"""
from __future__ import annotations

import ctypes as C
from typing import Any, Iterable, List, Optional, Sequence

import numpy as np

from . import _native as N

POSE_DTYPE = np.dtype([("rot", "<i4"), ("t_lin", "<i4"), ("score", "<f4"), ("flags", "<u4")])


class DockError(RuntimeError):
    def __init__(self, status: int, msg: str):
        super().__init__(f"{N.STATUS_NAMES.get(status, status)}: {msg}")
        self.status = status


def _torch():
    import torch
    return torch


def _is_torch(x) -> bool:
    try:
        import torch
        return isinstance(x, torch.Tensor)
    except ImportError:   # pragma: no cover
        return False


def _buf(x, dtype: str):
    """(pointer, keepalive) for a numpy array or torch tensor, contiguous, of the given dtype."""
    if x is None:
        return None, None
    if _is_torch(x):
        torch = _torch()
        tdt = {"f4": torch.float32, "f8": torch.float64, "i4": torch.int32}[dtype]
        t = x.detach()
        if t.dtype != tdt:
            t = t.to(tdt)
        t = t.contiguous()
        return t.data_ptr(), t
    a = np.ascontiguousarray(x, dtype={"f4": np.float32, "f8": np.float64, "i4": np.int32}[dtype])
    return a.ctypes.data, a


def _check(ctx_ptr, status: int):
    if status != N.DOCK_OK:
        msg = N.lib().dock_last_error(ctx_ptr) if ctx_ptr else b""
        raise DockError(status, (msg or b"").decode(errors="replace"))


class DockContext:
    """Owns a dock_ctx*.  Create with dock_init, release with dock_destroy (or ``close``)."""

    def __init__(self, ptr: int, P: int, n, m_max: int, device: int, stream_handle: int):
        self.ptr = C.c_void_p(ptr)
        self.P, self.n, self.m_max, self.device = P, tuple(n), m_max, device
        self.stream_handle = stream_handle

    @property
    def n_cells(self) -> int:
        return self.n[0] * self.n[1] * self.n[2]

    def close(self):
        if self.ptr:
            N.lib().dock_destroy(self.ptr)
            self.ptr = C.c_void_p(0)

    def __del__(self):  # pragma: no cover - best effort
        try:
            self.close()
        except Exception:
            pass


def dock_init(receptor, weights, spacing: float = 0.8, m_max: int = 8, device: int | None = None,
              stream=None) -> DockContext:
    """Copy receptor grids ``[P][nz][ny][nx]`` float32 and weights ``[P]`` to the device."""
    torch = _torch()
    shape = tuple(receptor.shape)
    if len(shape) != 4:
        raise ValueError("receptor must be [P][nz][ny][nx]")
    P, nz, ny, nx = shape
    if device is None:
        device = receptor.device.index if _is_torch(receptor) and receptor.is_cuda else torch.cuda.current_device()
    if stream is None:
        sh = torch.cuda.current_stream(device).cuda_stream
    elif isinstance(stream, int):
        sh = stream
    else:
        sh = stream.cuda_stream
    if sh == 0:
        # torch's default stream is the legacy default stream: pass cudaStreamLegacy (a NULL stream asks the
        # library to create a private one, which torch's work would not be ordered with)
        sh = 1
    rp, rk = _buf(receptor, "f4")
    wp, wk = _buf(weights, "f4")
    g = N.dock_grid_desc(nx, ny, nz, P, m_max, device, float(spacing), C.c_void_p(sh))
    out = C.c_void_p()
    with torch.cuda.device(device):
        st = N.lib().dock_init(C.byref(g), C.c_void_p(rp), C.c_void_p(wp), C.byref(out))
    _check(None, st)
    del rk, wk
    return DockContext(out.value, P, (nx, ny, nz), m_max, device, sh)


def _check_device(x, ctx: "DockContext", what: str):
    """torch CUDA tensors must live on the context's device (the C side also rejects other devices)."""
    if _is_torch(x) and x.is_cuda and x.device.index != ctx.device:
        raise ValueError(f"{what} is on cuda:{x.device.index}, the context is on cuda:{ctx.device}")


def _probe_array(probes: Sequence[Any], ctx: "DockContext"):
    keep: List[Any] = []
    arr = (N.dock_probe_desc * len(probes))()
    for i, p in enumerate(probes):
        xyz, coef, m = (p["xyz"], p["coef"], p["m"]) if isinstance(p, dict) else (p.xyz, p.coef, p.m)
        _check_device(xyz, ctx, f"probe {i} xyz")
        _check_device(coef, ctx, f"probe {i} coef")
        xp, xk = _buf(xyz, "f8")
        cp, ck = _buf(coef, "f4")
        keep += [xk, ck]
        n_atoms = int(xk.shape[0]) if xk.ndim >= 1 else 0
        # the C side reads n_atoms x 3 doubles and n_atoms x P floats: reject anything else here
        if tuple(xk.shape) != (n_atoms, 3):
            raise ValueError(f"probe {i}: xyz must be [n_atoms][3], got {tuple(xk.shape)}")
        if tuple(ck.shape) not in ((n_atoms, ctx.P),) and not (n_atoms == 0 and ck.size == 0):
            raise ValueError(f"probe {i}: coef must be [n_atoms][P] = [{n_atoms}][{ctx.P}], got {tuple(ck.shape)}")
        arr[i] = N.dock_probe_desc(n_atoms, int(m), C.c_void_p(xp if n_atoms else None),
                                   C.c_void_p(cp if n_atoms else None))
    return arr, keep


class ProbeSet:
    """Probes marshalled once into the C descriptor array (``dock_probe_desc[n]``) for repeated calls.

    ``dock_probe_batch`` marshals a plain probe list on every call (~5 us per probe in Python); a ProbeSet
    does it once.  It keeps the converted buffers alive: device tensors of the right dtype are referenced in
    place (later in-place updates are seen), anything that needed a dtype/layout conversion is a snapshot.
    """

    def __init__(self, ctx: "DockContext", probes: Sequence[Any]):
        self.arr, self._keep = _probe_array(probes, ctx)
        self.n = len(probes)
        self.P, self.device = ctx.P, ctx.device
        self.m = int(probes[0]["m"] if isinstance(probes[0], dict) else probes[0].m) if self.n else 0

    def __len__(self) -> int:
        return self.n


def dock_probes(ctx: "DockContext", probes: Sequence[Any]) -> ProbeSet:
    """Marshal a probe list once (see ProbeSet); pass the result to dock_probe_batch in place of the list."""
    return ProbeSet(ctx, probes)


def _alloc_poses(n_units: int, k: int, out, device: int):
    if out is None:
        o = np.zeros((n_units, k), dtype=POSE_DTYPE)
        return o, o.ctypes.data
    if _is_torch(out):
        if out.dtype != _torch().int32 or tuple(out.shape) != (n_units, k, 4) or not out.is_contiguous():
            raise ValueError("device pose buffer must be a contiguous int32 tensor [U][k][4]")
        if out.is_cuda and out.device.index != device:
            raise ValueError(f"pose buffer is on cuda:{out.device.index}, the context is on cuda:{device}")
        return out, out.data_ptr()
    if out.dtype != POSE_DTYPE or out.shape != (n_units, k) or not out.flags.c_contiguous:
        raise ValueError("host pose buffer must be a contiguous POSE_DTYPE array [U][k]")
    return out, out.ctypes.data


def dock_probe_batch(ctx: DockContext, probes: Sequence[Any], rot, unit_begin: int = 0,
                     unit_end: Optional[int] = None, k: int = 4, rho: int = 1, out=None):
    """Dock probe-major (probe, rotation) units [unit_begin, unit_end); the hot path.

    ``probes``: a sequence of probes ({"xyz", "coef", "m"} dicts or objects) or a ProbeSet (dock_probes).
    ``out``: None -> a host numpy POSE_DTYPE array [U][k] (synchronous); or a caller buffer (numpy
    POSE_DTYPE [U][k], synchronous; or an int32 torch tensor [U][k][4] on the context's device ->
    device-resident output, ASYNCHRONOUS: the call returns once the work is enqueued on the context's
    stream; call ``dock_sync`` for device-detected errors, see include/dock.h).
    """
    torch = _torch()
    n_rot = int(rot.shape[0])
    if unit_end is None:
        unit_end = len(probes) * n_rot
    _check_device(rot, ctx, "rot")
    rp, rk = _buf(rot, "f8")
    if isinstance(probes, ProbeSet):
        if probes.P != ctx.P or probes.device != ctx.device:
            raise ValueError("ProbeSet was built for another context (P or device differs)")
        arr, keep = probes.arr, None
    else:
        arr, keep = _probe_array(probes, ctx)
    o, op = _alloc_poses(unit_end - unit_begin, k, out, ctx.device)
    with torch.cuda.device(ctx.device):
        st = N.lib().dock_probe_batch(ctx.ptr, arr, len(probes), C.c_void_p(rp), n_rot, int(unit_begin),
                                      int(unit_end), int(k), int(rho), C.c_void_p(op))
    _check(ctx.ptr, st)
    del rk, keep
    return o


def dock_sync(ctx: DockContext):
    """Sync point of the asynchronous (device-output) calls: waits for the context's stream and raises
    DockError for a device-detected error of any call since the previous sync point."""
    torch = _torch()
    with torch.cuda.device(ctx.device):
        st = N.lib().dock_sync(ctx.ptr)
    _check(ctx.ptr, st)


def dock_probe(ctx: DockContext, probe, rot, k: int = 4, rho: int = 1, out=None):
    """Dock one probe over a rotation set -> poses [n_rot][k]."""
    return dock_probe_batch(ctx, [probe], rot, 0, int(rot.shape[0]), k, rho, out)


def dock_score_grid(ctx: DockContext, probe, rot9, per_term: bool = False):
    """Full weighted score grid S [nz][ny][nx] (and unweighted per-term C_p [P][nz][ny][nx])."""
    torch = _torch()
    nx, ny, nz = ctx.n
    S = np.zeros((nz, ny, nx), np.float32)
    C_ = np.zeros((ctx.P, nz, ny, nx), np.float32) if per_term else None
    rp, rk = _buf(np.asarray(rot9, dtype=np.float64).reshape(9) if not _is_torch(rot9) else rot9, "f8")
    arr, keep = _probe_array([probe], ctx)
    with torch.cuda.device(ctx.device):
        st = N.lib().dock_score_grid(ctx.ptr, arr, C.c_void_p(rp), C.c_void_p(S.ctypes.data),
                                     C.c_void_p(C_.ctypes.data if per_term else None))
    _check(ctx.ptr, st)
    return (S, C_) if per_term else S


def dock_voxelize(ctx: DockContext, probe, rot):
    """Unweighted voxelized probe grids L [n_rot][P][m][m][m] float32 (debug)."""
    torch = _torch()
    m = probe["m"] if isinstance(probe, dict) else probe.m
    n_rot = int(rot.shape[0])
    out = np.zeros((n_rot, ctx.P, m, m, m), np.float32)
    rp, rk = _buf(rot, "f8")
    arr, keep = _probe_array([probe], ctx)
    with torch.cuda.device(ctx.device):
        st = N.lib().dock_voxelize(ctx.ptr, arr, C.c_void_p(rp), n_rot, C.c_void_p(out.ctypes.data))
    _check(ctx.ptr, st)
    return out


def dock_set_tuning(ctx: DockContext, key: int, value: int):
    _check(ctx.ptr, N.lib().dock_set_tuning(ctx.ptr, int(key), int(value)))


def dock_get_info(ctx: DockContext) -> dict:
    info = N.dock_info()
    _check(ctx.ptr, N.lib().dock_get_info(ctx.ptr, C.byref(info)))
    return {f: getattr(info, f) for f, _ in N.dock_info._fields_}


def dock_destroy(ctx: DockContext):
    ctx.close()


def poses_from_device(t) -> np.ndarray:
    """int32 torch tensor [U][k][4] (device or host) -> numpy POSE_DTYPE [U][k]."""
    a = t.detach().cpu().contiguous().numpy()
    return a.view(POSE_DTYPE).reshape(a.shape[:-1])
