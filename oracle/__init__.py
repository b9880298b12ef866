"""FP64 CPU oracle for the rigid-docking hot path -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py`` (its ``cpu_baseline``
leg and ``--impl reference``) may import this package.  The product path
(``paper_conf_ipps_sukhwanih10_b200``) never imports it and shares no code with it.

``dock_oracle.c`` holds the arithmetic (voxelize / score / filter / dock, each citing
PAPER.md); this module only compiles it and marshals numpy arrays through ctypes.
Parity status: every function is pinned by tests/test_oracle_pins.py (see DESIGN.md
§"Oracle pins").
"""
from .oracle import (  # noqa: F401
    build_oracle, check_rotation, voxelize, score_grid, filter_greedy, dock,
    max_threads, OracleError,
)
from .em import build_em_oracle, em_eval  # noqa: F401  (EM non-bonded energy, NEXT-4)
