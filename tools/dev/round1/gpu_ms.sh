#!/bin/bash
# dev helper (under gpurun): shared-adjacency multi-source push -- parity, microbench, benches
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 300 python -m pytest tests -m gpu -x -q --timeout 200 -k "shared" > gpurun_out/pytest_shared.log 2>&1; echo pytest-shared rc=$?; tail -3 gpurun_out/pytest_shared.log
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/msab tools/ms_atomic_bench.cu && timeout 120 /tmp/msab > gpurun_out/ms_atomic_bench.txt 2>&1; cat gpurun_out/ms_atomic_bench.txt
export CFGFILE=tools/cfgs_ms_shared.sh
bash tools/bench_configs.sh
