#!/bin/bash
# compute-sanitizer memcheck + racecheck on the GPU parity tests (under gpurun)
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
K1="fig or empty or enoent or erange or cancels or multiset or tiny_config_all_modes or shared or multi_source or schedules"
K2="fig2 or tiny_config_all_modes or tiny_config_multi_source_shared or schedules"
timeout 2400 compute-sanitizer --tool memcheck python -m pytest tests/test_gpu_parity.py -m gpu -q -k "$K1" > gpurun_out/san_memcheck.log 2>&1; echo memcheck rc=$?; tail -3 gpurun_out/san_memcheck.log
timeout 2400 compute-sanitizer --tool racecheck python -m pytest tests/test_gpu_parity.py -m gpu -q -k "$K2" > gpurun_out/san_racecheck.log 2>&1; echo racecheck rc=$?; tail -3 gpurun_out/san_racecheck.log
