"""Tie-aware pose validator.

GPU picks are compared with the FP64 oracle's score grid S and magnitude grid A:
  * pick j must be available after GPU picks 1..j-1 (cyclic Chebyshev exclusion, radius rho);
  * S(pick_j) <= min over available cells of S + tol * max(A(pick_j), A(best)), i.e. the
    GPU may only deviate from the oracle's choice inside the FP32 tolerance band;
  * the reported FP32 score is within tol * A(pick_j) of S(pick_j).
Indices therefore agree bit-exactly whenever the oracle's competing gap exceeds the band.
"""
from __future__ import annotations

import numpy as np


def _exclude(avail: np.ndarray, t: int, rho: int, shape):
    nz, ny, nx = shape
    x, y, z = t % nx, (t // nx) % ny, t // (nx * ny)
    xs = [(x + d) % nx for d in range(-rho, rho + 1)]
    ys = [(y + d) % ny for d in range(-rho, rho + 1)]
    zs = [(z + d) % nz for d in range(-rho, rho + 1)]
    a = avail.reshape(shape)
    a[np.ix_(zs, ys, xs)] = False


def validate_unit(S: np.ndarray, A: np.ndarray, gpu_t, gpu_s, k: int, rho: int, tol: float = 1e-4):
    """Raise AssertionError on a violation; return the number of picks whose index differs
    from the oracle's own choice (only possible inside the tolerance band)."""
    Sf, Af = S.reshape(-1), A.reshape(-1)
    avail = np.ones(Sf.size, dtype=bool)
    mism = 0
    for j in range(k):
        t = int(gpu_t[j])
        assert 0 <= t < Sf.size, f"pick {j}: t_lin {t} out of range"
        assert avail[t], f"pick {j}: t_lin {t} was excluded by an earlier pick"
        idx = np.flatnonzero(avail)
        Sa = Sf[idx]
        smin = Sa.min()
        best = int(idx[np.flatnonzero(Sa == smin)[0]])          # oracle key: (score, t_lin)
        band = tol * max(Af[t], Af[best]) + 1e-12
        assert Sf[t] - Sf[best] <= band, (
            f"pick {j}: S[{t}]={Sf[t]!r} exceeds best available S[{best}]={Sf[best]!r} by more than {band!r}")
        assert abs(float(gpu_s[j]) - Sf[t]) <= tol * Af[t] + 1e-12, (
            f"pick {j}: reported score {gpu_s[j]!r} vs oracle {Sf[t]!r} (A={Af[t]!r})")
        mism += int(t != best)
        _exclude(avail, t, rho, S.shape)
    return mism
