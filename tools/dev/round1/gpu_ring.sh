#!/bin/bash
# ring-worklist flush policy: parity + A/B of build/variants on the ring-heavy configs (under gpurun)
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 900 python -m pytest tests -m gpu -q -x --timeout 600 -k "schedules or all_modes or orkut or undirected or lj_full" > gpurun_out/pytest_ring.log 2>&1; echo pytest rc=$?; tail -2 gpurun_out/pytest_ring.log
BENCH_ARGS="--workload orkut --steps 10" bash tools/ab_variants.sh
BENCH_ARGS="" bash tools/ab_variants.sh
BENCH_ARGS="--mode async" bash tools/ab_variants.sh
BENCH_ARGS="--workload twitter --steps 4" bash tools/ab_variants.sh
BENCH_ARGS="--workload orkut --steps 10" bash tools/ab_variants.sh
