#!/bin/bash
# sparse-engine GPU check: parity tests of engine 4 + bench lines per config (run under gpurun)
python -c "import __graft_entry__ as e; e.build()" || exit 1
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "${TESTK:-4}" 2>&1 | tail -8
for c in prod c64; do
  for e in ${ENGINES:-sparse tc}; do
    timeout 300 python bench.py --config $c --engine $e --steps 5 --warmup 3 --no-cpu-baseline --no-alt --no-e2e > gpurun_out/b_${c}_$e.json 2>gpurun_out/b_${c}_$e.err || tail -c 800 gpurun_out/b_${c}_$e.err
  done
done
timeout 300 python bench.py --config large --rotations 8750 --engine sparse --steps 3 --warmup 3 --no-cpu-baseline --no-alt --no-e2e > gpurun_out/b_large_sparse.json 2>gpurun_out/b_large_sparse.err || tail -c 800 gpurun_out/b_large_sparse.err
python - <<'PY'
import json, glob
for f in sorted(glob.glob("gpurun_out/b_*.json")):
    try:
        d = json.load(open(f)); r = d["roofline"]
        print(f, round(d["value"]), "ms/step %.3f pipelined %.3f" % (d["ms_per_step"], d.get("ms_per_step_pipelined", -1)),
              "kernel_ms", r.get("launch_ms"), "frac %.3f" % r["frac"], r["bound"], "fb", d["config"]["fallback_rotations"])
    except Exception as e:
        print(f, "ERR", e)
PY
