#!/bin/bash
mkdir -p gpurun_out/r2c
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 2400 python -m pytest tests -m gpu -q --timeout 900 > gpurun_out/r2c/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/r2c/pytest_gpu.log
timeout 600 python bench.py --workload tiny --no-multi-source > gpurun_out/r2c/cfg_tiny.json 2> gpurun_out/r2c/cfg_tiny.err; echo tiny rc=$?
REPS=2 PARITY_K="test_tiny_config_all_modes_track_oracle and opt" BENCH_ARGS="--no-multi-source" bash tools/dev/gpu_ab.sh
