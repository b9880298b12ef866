#!/bin/bash
# Round-2 evidence (run under gpurun, 1 GPU): bench lines (prod = the headline, c64, the large config's
# per-rank shard), the ncu launch list of the prod bench command, and one ncu --set full capture of the
# dominant kernel of prod (k_corr_tc) and of the large shard (k_corr_sparse).
set -u
mkdir -p gpurun_out
TAG=${1:-r02}
python -c "import __graft_entry__ as e; e.build()" > gpurun_out/build_${TAG}.log 2>&1 || { tail gpurun_out/build_${TAG}.log; exit 1; }
echo "== bench prod"; timeout 900 python bench.py > gpurun_out/bench_${TAG}_prod.json 2> gpurun_out/bench_${TAG}_prod.err; echo "rc=$?"
echo "== bench c64"; timeout 600 python bench.py --config c64 --no-cpu-baseline > gpurun_out/bench_${TAG}_c64.json 2> gpurun_out/bench_${TAG}_c64.err; echo "rc=$?"
echo "== bench large shard"; timeout 900 python bench.py --config large --rotations 8750 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/bench_${TAG}_large.json 2> gpurun_out/bench_${TAG}_large.err; echo "rc=$?"
echo "== shard times (single-GPU projection input)"; timeout 600 python scripts/shard_times.py > gpurun_out/shard_times_${TAG}_prod.json; timeout 900 python scripts/shard_times.py --config large --rotations 8750 --steps 3 > gpurun_out/shard_times_${TAG}_large.json; tail -c 400 gpurun_out/shard_times_${TAG}_prod.json
echo "== host gaps"; python scripts/host_gaps.py > gpurun_out/host_gaps_${TAG}.json
echo "== EM bench"; python scripts/bench_em.py > gpurun_out/em_bench_${TAG}.json
echo "== launch list prod"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_${TAG}_prod.csv \
    python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --no-alt > gpurun_out/launches_${TAG}_prod.log 2>&1; echo "rc=$?"
echo "== full capture k_corr_tc (prod)"; SKIP=1 bash scripts/ncu_kernel.sh ${TAG}_prod_tc k_corr_tc --config prod --engine tc
echo "== full capture k_corr_sparse (c64 bench launch)"; SKIP=1 bash scripts/ncu_kernel.sh ${TAG}_c64_sparse k_corr_sparse --config c64
echo "== full capture k_corr_sparse (large shard bench launch, 8750 rotations)"; SKIP=1 bash scripts/ncu_kernel.sh ${TAG}_large_sparse k_corr_sparse --config large --rotations 8750
ls gpurun_out | head -50
