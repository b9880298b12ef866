#!/usr/bin/env python
"""Full-workload oracle results for the GPU parity tests (TEST INFRASTRUCTURE; calls only oracle/).

For a BASELINE config this docks EVERY (probe, rotation) unit with the FP64 oracle (oracle/dock_oracle.c)
and stores, per unit, the k picks (t_lin), their FP64 scores S and magnitude sums A (reading Q16) and the
status, keyed by a hash of the generated inputs (dockgen, seeded).  tests/test_gpu_full_parity.py compares
the GPU's poses on the same inputs unit by unit; a unit whose picks differ is re-scored in full with the
oracle and checked by the tie-aware validator.  No value here comes from the CUDA path.

    python scripts/oracle_cache.py --config prod   # ~8.6 TFLOP of FP64: ~30-40 min on 8 cores
    python scripts/oracle_cache.py --config c64
"""
from __future__ import annotations

import argparse
import hashlib
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402

import dockgen as g  # noqa: E402

GOLDEN = os.path.join(ROOT, "tests", "golden")


def inputs(cfg: str):
    c = g.CONFIGS[cfg]
    R = g.receptor_ftmap_like(c.n, c.P)
    w = g.weights(c.P)
    probes = g.probes(c.n_probes, c.m, c.P)
    rot = g.rotations(c.n_rot)
    return c, R, w, probes, rot


def input_hash(R, w, probes, rot, k: int, rho: int) -> str:
    h = hashlib.sha256()
    for a in [R, w, rot] + [p.xyz for p in probes] + [p.coef for p in probes]:
        a = np.ascontiguousarray(a)
        h.update(str(a.dtype).encode() + str(a.shape).encode())
        h.update(a.tobytes())
    h.update(f"m={[p.m for p in probes]} h={g.SPACING!r} k={k} rho={rho}".encode())
    return h.hexdigest()


def cache_path(cfg: str, k: int, rho: int) -> str:
    return os.path.join(GOLDEN, f"oracle_{cfg}_k{k}_rho{rho}.npz")


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="prod", choices=["c64", "prod"])
    ap.add_argument("--rho", type=int, default=1)
    ap.add_argument("--chunk", type=int, default=64)
    args = ap.parse_args()
    import oracle
    oracle.build_oracle()
    c, R, w, probes, rot = inputs(args.config)
    k = c.k
    n = c.n_probes * c.n_rot
    t = np.full((n, k), -1, np.int64)
    s = np.full((n, k), np.nan)
    a = np.full((n, k), np.nan)
    st = np.zeros(n, np.int32)
    t0 = time.time()
    for b in range(0, n, args.chunk):
        e = min(n, b + args.chunk)
        t[b:e], s[b:e], st[b:e], a[b:e] = oracle.dock(R, w, g.SPACING, probes, rot, k, args.rho,
                                                      unit_begin=b, unit_end=e, with_A=True)
        print(f"{args.config}: {e}/{n} units, {time.time() - t0:.0f} s", flush=True)
    os.makedirs(GOLDEN, exist_ok=True)
    path = cache_path(args.config, k, args.rho)
    np.savez_compressed(path, t_lin=t, score=s, A=a, status=st,
                        input_hash=np.array(input_hash(R, w, probes, rot, k, args.rho)),
                        note=np.array(f"FP64 oracle (oracle/dock_oracle.c), config {args.config}, k={k}, "
                                      f"rho={args.rho}, written by scripts/oracle_cache.py"))
    print(f"wrote {path} ({time.time() - t0:.0f} s)")


if __name__ == "__main__":
    main()
