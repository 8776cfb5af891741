#!/bin/bash
mkdir -p gpurun_out/chk3
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 2400 python -m pytest tests -m gpu -q --timeout 900 > gpurun_out/chk3/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/chk3/pytest_gpu.log
REPS=2 PARITY_K="test_tiny_config_all_modes_track_oracle and opt or test_opt_schedules" BENCH_ARGS="--no-multi-source" bash tools/dev/gpu_ab.sh
PPR_TRACE=1 timeout 300 python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e --no-multi-source > gpurun_out/chk3/trace.json 2> gpurun_out/chk3/trace.err; echo trace rc=$?
