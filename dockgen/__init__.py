"""Seeded synthetic input generators shared by the oracle tests and the CUDA path.

This module holds NONE of the docking method's arithmetic (no voxelization,
no correlation, no scoring, no filtering).  It only manufactures inputs with
the shapes and statistics of FTMap's rigid-docking workload:

* receptor grids  R_p, float32 ``[P][nz][ny][nx]`` (x fastest)   -- PAPER.md L140-141, L533-545
* probes          atoms ``xyz [n][3]`` float64 (Å, relative to the centroid)
                  and per-atom, per-term coefficients ``coef [n][P]`` float32
                                                                  -- PAPER.md L184-186, L544-555
* rotation sets   proper rotation matrices ``[R][9]`` float64, row-major
                                                                  -- PAPER.md L162-166
* term weights    ``w [P]`` float32 (Eq. 2, flattened per channel) -- PAPER.md L173-183

Everything is drawn from ``numpy.random.default_rng(seed)`` (PCG64), so the two
sides of a parity test see bit-identical inputs.  The recipe is stated in
DESIGN.md §"Input recipe".
"""
from __future__ import annotations

import math
from dataclasses import dataclass
from typing import List, Sequence, Tuple

import numpy as np

SPACING = 0.8  # Å per voxel (BASELINE.json configs; the paper never states it)
N_TYPES = 18   # receptor / probe atom types

# --------------------------------------------------------------------------- rotations


def quat_to_matrix(q: np.ndarray) -> np.ndarray:
    """Unit quaternion(s) (w, x, y, z) -> row-major 3x3 rotation matrices, float64."""
    q = np.asarray(q, dtype=np.float64)
    q = q / np.linalg.norm(q, axis=-1, keepdims=True)
    w, x, y, z = q[..., 0], q[..., 1], q[..., 2], q[..., 3]
    m = np.empty(q.shape[:-1] + (3, 3), dtype=np.float64)
    m[..., 0, 0] = 1 - 2 * (y * y + z * z)
    m[..., 0, 1] = 2 * (x * y - w * z)
    m[..., 0, 2] = 2 * (x * z + w * y)
    m[..., 1, 0] = 2 * (x * y + w * z)
    m[..., 1, 1] = 1 - 2 * (x * x + z * z)
    m[..., 1, 2] = 2 * (y * z - w * x)
    m[..., 2, 0] = 2 * (x * z - w * y)
    m[..., 2, 1] = 2 * (y * z + w * x)
    m[..., 2, 2] = 1 - 2 * (x * x + y * y)
    return m


def shoemake_quaternions(n: int, seed: int) -> np.ndarray:
    """n Shoemake-uniform unit quaternions, sign-canonical (w >= 0)."""
    rng = np.random.default_rng(seed)
    u1, u2, u3 = rng.random(n), rng.random(n), rng.random(n)
    a, b = np.sqrt(1.0 - u1), np.sqrt(u1)
    q = np.stack([b * np.cos(2 * np.pi * u3), a * np.sin(2 * np.pi * u2),
                  a * np.cos(2 * np.pi * u2), b * np.sin(2 * np.pi * u3)], axis=1)
    q[q[:, 0] < 0] *= -1.0
    return q


def cube_group() -> np.ndarray:
    """The 24 proper rotations of the cube (signed permutation matrices, det = +1), [24][9]."""
    out = []
    import itertools
    for perm in itertools.permutations(range(3)):
        for signs in itertools.product((1.0, -1.0), repeat=3):
            m = np.zeros((3, 3))
            for i in range(3):
                m[i, perm[i]] = signs[i]
            if np.linalg.det(m) > 0:
                out.append(m.reshape(9))
    return np.array(out, dtype=np.float64)


def rotations(n: int, seed: int = 3001, with_cube_group: bool = False) -> np.ndarray:
    """Rotation set ``[n][9]`` float64: index 0 = identity, the rest Shoemake-uniform.

    With ``with_cube_group`` the 24 cube-group rotations are appended (test sets).
    """
    if n < 1:
        mats = np.zeros((0, 9))
    else:
        q = shoemake_quaternions(n, seed)
        q[0] = (1.0, 0.0, 0.0, 0.0)
        mats = quat_to_matrix(q).reshape(n, 9)
    if with_cube_group:
        mats = np.concatenate([mats, cube_group()], axis=0)
    return np.ascontiguousarray(mats, dtype=np.float64)


# --------------------------------------------------------------------------- weights


def channel_names(P: int) -> List[str]:
    """Channel (term) names for P correlation terms (Eq. 2 flattened)."""
    if P == 1:
        return ["shape"]
    if P == 2:
        return ["attr", "rep"]
    if P == 3:
        return ["attr", "rep", "elec"]
    if P == 4:
        return ["attr", "rep", "elec", "desolv0"]
    return ["attr", "rep", "elec_short", "elec_long"] + [f"desolv{i}" for i in range(P - 4)]


_W = {"shape": 1.0, "attr": 1.0, "rep": 1.0, "elec": 0.6, "elec_short": 0.6, "elec_long": 0.6}


def weights(P: int) -> np.ndarray:
    """Synthetic Eq. 2 term weights (the paper gives none): shape 1, elec 0.6, desolv 0.4."""
    return np.array([_W.get(c, 0.4) for c in channel_names(P)], dtype=np.float32)


def weights_integer(P: int, seed: int = 4001) -> np.ndarray:
    """Weights from {1, 2, 1/2} (exactly representable; integer-input pin P9)."""
    rng = np.random.default_rng(seed)
    return rng.choice(np.array([1.0, 2.0, 0.5], dtype=np.float32), size=P)


# --------------------------------------------------------------------------- receptors


def receptor_uniform(n: Sequence[int], P: int, seed: int = 1002) -> np.ndarray:
    """iid U(-1, 1) receptor channels, ``[P][nz][ny][nx]`` float32 (ties rare; stress)."""
    nx, ny, nz = n
    rng = np.random.default_rng(seed)
    return rng.uniform(-1.0, 1.0, size=(P, nz, ny, nx)).astype(np.float32)


def receptor_integer(n: Sequence[int], P: int, seed: int = 1003, lo: int = -8, hi: int = 8) -> np.ndarray:
    """iid integers in [lo, hi] (exact in fp32 products/sums; many exact ties)."""
    nx, ny, nz = n
    rng = np.random.default_rng(seed)
    return rng.integers(lo, hi + 1, size=(P, nz, ny, nx)).astype(np.float32)


@dataclass
class Protein:
    xyz: np.ndarray     # [A][3] Å, box coordinates
    types: np.ndarray   # [A] int
    charge: np.ndarray  # [A] float


def protein_atoms(n: Sequence[int], spacing: float = SPACING, seed: int = 1001) -> Protein:
    """~2200 heavy atoms (density 0.05 Å^-3) uniform in a sphere of radius <= 22 Å at the box centre."""
    nx, ny, nz = n
    box = np.array([nx, ny, nz], dtype=np.float64) * spacing
    radius = min(22.0, 0.35 * float(box.min()))
    n_atoms = max(8, int(round(0.05 * 4.0 / 3.0 * math.pi * radius ** 3)))
    rng = np.random.default_rng(seed)
    d = rng.normal(size=(n_atoms, 3))
    d /= np.linalg.norm(d, axis=1, keepdims=True)
    r = radius * rng.random(n_atoms) ** (1.0 / 3.0)
    xyz = box / 2.0 + d * r[:, None]
    types = rng.integers(0, N_TYPES, size=n_atoms)
    charge = rng.uniform(-0.5, 0.5, size=n_atoms)
    return Protein(xyz=xyz, types=types, charge=charge)


def _offsets(cut_vox: int) -> np.ndarray:
    r = np.arange(-cut_vox, cut_vox + 1)
    oz, oy, ox = np.meshgrid(r, r, r, indexing="ij")
    return np.stack([ox.ravel(), oy.ravel(), oz.ravel()], axis=1)


def _splat(prot: Protein, n: Sequence[int], spacing: float, cutoff: float, chunk: int = 192):
    """Yield (flat voxel index, distance Å, atom index) for voxel/atom pairs with d < cutoff.

    Voxel (i, j, k) has its centre at (i, j, k) * spacing; indices wrap cyclically
    (the protein sits well inside the box, so wrapping never matters in practice).
    """
    nx, ny, nz = n
    cv = int(math.ceil(cutoff / spacing)) + 1
    off = _offsets(cv)
    # only offsets that can reach within the cutoff of an atom inside its base voxel
    off = off[np.linalg.norm(off, axis=1) * spacing <= cutoff + spacing * math.sqrt(3.0)]
    base = np.floor(prot.xyz / spacing).astype(np.int64)
    for a0 in range(0, len(prot.xyz), chunk):
        a1 = min(len(prot.xyz), a0 + chunk)
        cells = base[a0:a1, None, :] + off[None, :, :]           # [c][K][3]
        d = np.linalg.norm(cells * spacing - prot.xyz[a0:a1, None, :], axis=2)
        keep = d < cutoff
        c = cells[keep]
        flat = ((c[:, 2] % nz) * ny + (c[:, 1] % ny)) * nx + (c[:, 0] % nx)
        atom = np.broadcast_to(np.arange(a0, a1)[:, None], keep.shape)[keep]
        yield flat, d[keep], atom


def receptor_ftmap_like(n: Sequence[int], P: int, spacing: float = SPACING, seed: int = 1001) -> np.ndarray:
    """FTMap-like receptor channels ``[P][nz][ny][nx]`` float32 (recipe: DESIGN.md).

    attr = -1 on the shell 1.8 Å < d_min < 5.2 Å, else 0; rep = #atoms with d < 1.8 Å;
    elec = clip(sum q / (4 max(d,1)^2), +-5) (short: d < 6 Å, long: 6 <= d < 12 Å);
    desolv_p = sum u[p, type] [d < 6 Å], u ~ N(0, 1).
    """
    nx, ny, nz = n
    nv = nx * ny * nz
    prot = protein_atoms(n, spacing, seed)
    rng = np.random.default_rng(seed + 7)
    names = channel_names(P)
    n_des = sum(1 for c in names if c.startswith("desolv"))
    u = rng.normal(size=(max(n_des, 1), N_TYPES))

    near = np.zeros(nv)       # atoms within 1.8 Å
    shell = np.zeros(nv)      # atoms within 5.2 Å
    e_short = np.zeros(nv)
    e_long = np.zeros(nv)
    des = np.zeros((max(n_des, 1), nv))
    for flat, d, atom in _splat(prot, n, spacing, 12.0):
        e = prot.charge[atom] / (4.0 * np.maximum(d, 1.0) ** 2)
        s = d < 6.0
        e_short += np.bincount(flat[s], weights=e[s], minlength=nv)
        e_long += np.bincount(flat[~s], weights=e[~s], minlength=nv)
        near += np.bincount(flat[d < 1.8], minlength=nv)
        shell += np.bincount(flat[d < 5.2], minlength=nv)
        for q in range(n_des):
            des[q] += np.bincount(flat[s], weights=u[q, prot.types[atom[s]]], minlength=nv)
    attr = np.where((near == 0) & (shell > 0), -1.0, 0.0)
    chans = {
        "attr": attr, "rep": near, "shape": attr + near,
        "elec": np.clip(e_short + e_long, -5, 5),
        "elec_short": np.clip(e_short, -5, 5), "elec_long": np.clip(e_long, -5, 5),
    }
    for q in range(n_des):
        chans[f"desolv{q}"] = des[q]
    out = np.stack([chans[c] for c in names]).reshape(P, nz, ny, nx)
    return np.ascontiguousarray(out, dtype=np.float32)


def receptor(kind: str, n: Sequence[int], P: int, seed: int | None = None) -> np.ndarray:
    if kind == "ftmap":
        return receptor_ftmap_like(n, P, seed=1001 if seed is None else seed)
    if kind == "uniform":
        return receptor_uniform(n, P, seed=1002 if seed is None else seed)
    if kind == "integer":
        return receptor_integer(n, P, seed=1003 if seed is None else seed)
    raise ValueError(kind)


# --------------------------------------------------------------------------- probes


@dataclass
class Probe:
    xyz: np.ndarray   # [n][3] float64, Å relative to the rotation centre (centroid)
    coef: np.ndarray  # [n][P] float32
    m: int            # probe grid edge (voxels)

    @property
    def n_atoms(self) -> int:
        return int(self.xyz.shape[0])


def probe(i: int, m: int, P: int, spacing: float = SPACING, seed: int | None = None,
          n_atoms: int | None = None, integer: bool = False) -> Probe:
    """FTMap-like probe ``i``: 2 + (i mod 7) heavy atoms, every rotation inside the m^3 box.

    Atoms are placed (rejection sampling, min separation ~1.0 Å when it fits) so that
    |x| < (m/2)*spacing - 0.05 Å after re-centring on the centroid; hence the nearest
    voxel of every rotated atom lies inside [0, m)^3.  coef: attr = rep = shape = 1,
    elec = q ~ U(-0.6, 0.6) re-centred to sum 0, desolv from a seeded type table.
    ``integer`` draws integer coefficients in [-4, 4] instead (pin P9).
    """
    rng = np.random.default_rng(2001 + i if seed is None else seed)
    n = n_atoms if n_atoms is not None else 2 + (i % 7)
    rmax = (m / 2.0) * spacing - 0.05
    sep = min(1.0, 0.9 * rmax)
    xyz = None
    for attempt in range(20000):
        d = rng.normal(size=(n, 3))
        d /= np.linalg.norm(d, axis=1, keepdims=True)
        x = d * (rmax * rng.random(n) ** (1.0 / 3.0))[:, None]
        x -= x.mean(axis=0)
        if np.max(np.linalg.norm(x, axis=1)) >= rmax:
            continue
        if n > 1:
            dd = np.linalg.norm(x[:, None] - x[None, :], axis=2) + np.eye(n) * 1e9
            if dd.min() < sep:
                if attempt % 2000 == 1999:
                    sep *= 0.8
                continue
        xyz = x
        break
    if xyz is None:
        raise RuntimeError("probe placement failed")
    if integer:
        coef = rng.integers(-4, 5, size=(n, P)).astype(np.float32)
    else:
        names = channel_names(P)
        types = rng.integers(0, N_TYPES, size=n)
        table = np.random.default_rng(5001).normal(scale=0.5, size=(P, N_TYPES))
        q = rng.uniform(-0.6, 0.6, size=n)
        q -= q.mean()
        coef = np.zeros((n, P), dtype=np.float64)
        for p, c in enumerate(names):
            if c in ("attr", "rep", "shape"):
                coef[:, p] = 1.0
            elif c.startswith("elec"):
                coef[:, p] = q
            else:
                coef[:, p] = table[p, types]
        coef = coef.astype(np.float32)
    return Probe(xyz=np.ascontiguousarray(xyz, dtype=np.float64),
                 coef=np.ascontiguousarray(coef, dtype=np.float32), m=m)


def probes(n_probes: int, m: int, P: int, spacing: float = SPACING, integer: bool = False) -> List[Probe]:
    return [probe(i, m, P, spacing, integer=integer) for i in range(n_probes)]


def voxel_centre_probe(cells: Sequence[Tuple[int, int, int]], m: int, P: int, spacing: float = SPACING,
                       coef: np.ndarray | None = None) -> Probe:
    """Probe with one atom exactly on each given voxel centre (vx, vy, vz) of the m^3 box."""
    c = (m - 1) / 2.0
    xyz = np.array([[(vx - c) * spacing, (vy - c) * spacing, (vz - c) * spacing] for vx, vy, vz in cells],
                   dtype=np.float64).reshape(-1, 3)
    if coef is None:
        coef = np.ones((len(cells), P), dtype=np.float32)
    return Probe(xyz=xyz, coef=np.ascontiguousarray(coef, dtype=np.float32), m=m)


# --------------------------------------------------------------------------- configs (BASELINE.json)


@dataclass
class Config:
    name: str
    n: Tuple[int, int, int]
    m: int
    P: int
    n_rot: int
    n_probes: int
    k: int
    rho: int = 1
    receptor_kind: str = "ftmap"


CONFIGS = {
    "toy": Config("toy", (32, 32, 32), 4, 1, 8, 1, 1),
    "c64": Config("c64", (64, 64, 64), 5, 4, 500, 1, 4),
    "prod": Config("prod", (128, 128, 128), 4, 4, 500, 16, 4),
    "large": Config("large", (160, 160, 160), 8, 22, 70000, 1, 4),
}


# --------------------------------------------------------------------------- energy minimisation (NEXT-4)


@dataclass
class EmSystem:
    """Synthetic non-bonded system of FTMap's energy minimisation (§II.B; parameters are synthetic:
    the paper gives none and CHARMM parameters are out of scope).  Pairs i < j within rc of the reference
    coordinates (the neighbour list the paper keeps fixed over many iterations)."""
    x0: np.ndarray      # [n][3] reference coordinates (A)
    q: np.ndarray       # [n] charges (e)
    R: np.ndarray       # [n] intrinsic radii (A)
    V: np.ndarray       # [n] solute volumes (A^3)
    eps: np.ndarray     # [n] vdW well depths
    rm: np.ndarray      # [n] vdW radii (rm_i; rm_ij = (rm_i + rm_j)/2)
    type: np.ndarray    # [n] atom types
    omega: np.ndarray   # [T][T] ACE Gaussian heights (ordered type pair)
    sigma: np.ndarray   # [T][T] ACE Gaussian widths
    mu: np.ndarray      # [T][T] ACE atom-atom parameters
    pairs: np.ndarray   # [n_pairs][2] int32, i < j, sorted by (i, j)
    eps_s: float = 80.0
    rc: float = 9.0


def em_system(n_atoms: int = 2200, seed: int = 5001, rc: float = 9.0, spacing: float = 2.7) -> EmSystem:
    """~n_atoms atoms on a jittered cubic lattice (min separation > 2 A) inside a sphere (protein-like density)."""
    rng = np.random.default_rng(seed)
    side = int(np.ceil((n_atoms * 6.0 / np.pi) ** (1.0 / 3.0))) + 2
    g = np.arange(side) * spacing
    pts = np.stack(np.meshgrid(g, g, g, indexing="ij"), -1).reshape(-1, 3)
    c = pts.mean(0)
    pts = pts[np.argsort(np.linalg.norm(pts - c, axis=1), kind="stable")[:n_atoms]]
    x0 = pts + rng.uniform(-0.3, 0.3, size=pts.shape)
    T = 6
    typ = rng.integers(0, T, size=n_atoms).astype(np.int32)
    d = np.linalg.norm(x0[:, None, :] - x0[None, :, :], axis=2)
    i, j = np.nonzero(np.triu(d < rc, k=1))
    pairs = np.stack([i, j], 1).astype(np.int32)
    return EmSystem(x0=x0, q=rng.uniform(-0.5, 0.5, n_atoms), R=rng.uniform(1.4, 2.0, n_atoms),
                    V=rng.uniform(10.0, 30.0, n_atoms), eps=rng.uniform(0.05, 0.2, n_atoms),
                    rm=rng.uniform(1.7, 2.2, n_atoms), type=typ, omega=rng.uniform(0.0, 0.02, (T, T)),
                    sigma=rng.uniform(2.5, 4.0, (T, T)), mu=rng.uniform(1.5, 3.0, (T, T)), pairs=pairs, rc=rc)


def em_conformations(s: EmSystem, n_conf: int, seed: int = 5002, jitter: float = 0.05) -> np.ndarray:
    """n_conf conformations [n_conf][n][3]: the reference plus small Gaussian displacements (minimisation
    moves atoms by small amounts)."""
    rng = np.random.default_rng(seed)
    return s.x0[None] + rng.normal(0.0, jitter, size=(n_conf,) + s.x0.shape)
