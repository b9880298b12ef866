#!/usr/bin/env python
"""Benchmark of the energy-minimisation non-bonded kernels (include/dock_em.h).

Workload: a protein-sized synthetic system (2200 atoms; pairs within a 9 A cut-off, fixed
over the evaluations as the paper's neighbour lists are) and a batch of conformations (the
2000 docked poses of a probe are minimised independently).  One step = energies + forces of
the whole batch (the paper's kernels (a)-(c)).  Prints one JSON line: conformation
evaluations/s, pair interactions/s, the paper's per-iteration GPU time (Table 2, C1060) for context, and
the FP64 oracle on the host cores.  python scripts/bench_em.py [--atoms 2200] [--conf 256] [--steps 10]
"""
import argparse
import json
import os
import statistics
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402

import dockgen as g  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--atoms", type=int, default=2200)
    ap.add_argument("--conf", type=int, default=256)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    args = ap.parse_args()
    import torch
    import paper_conf_ipps_sukhwanih10_b200 as D
    s = g.em_system(args.atoms)
    x = torch.from_numpy(g.em_conformations(s, args.conf)).cuda()
    ctx = D.em.em_init(s)
    for _ in range(args.warmup):
        D.em.em_eval(ctx, x)
    ms = []
    for _ in range(args.steps):
        D.em.em_eval(ctx, x)
        ms.append(D.em.em_last_ms(ctx))
    t = statistics.median(ms)
    n_pairs = int(s.pairs.shape[0])
    import oracle
    xc = g.em_conformations(s, 4)
    t0 = time.perf_counter()
    oracle.em_eval(s, xc, n_threads=len(os.sched_getaffinity(0)))
    tc = (time.perf_counter() - t0) / 4
    line = {"metric": "energy-minimisation non-bonded evaluations (energies + forces) per second",
            "value": args.conf / (t / 1e3), "unit": "conformation evaluations/s",
            "pair_interactions_per_s": args.conf * n_pairs / (t / 1e3), "ms_per_step": t,
            "ms_per_step_min": min(ms), "steps": args.steps, "warmup": args.warmup, "dtype": "f64",
            "config": {"atoms": args.atoms, "pairs": n_pairs, "conformations": args.conf, "cutoff_A": s.rc,
                       "kernels": "k_em_self, k_em_pair, k_em_chain, k_em_force, k_em_energy"},
            "paper_context": "Table 2 (P:L1162-1169): 0.23 + 2 x 0.19 + 0.14 ms per iteration of ~2200 atoms on a "
                             "Tesla C1060 = 1.3k evaluations/s",
            "cpu_baseline": {"value": 1.0 / tc, "unit": "conformation evaluations/s", "kind": "oracle",
                             "cores": len(os.sched_getaffinity(0)), "sample": "4 conformations, FP64 C oracle"}}
    print(json.dumps(line), flush=True)
    ctx.close()


if __name__ == "__main__":
    main()
