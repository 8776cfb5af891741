#!/bin/bash
mkdir -p gpurun_out/r2b
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -q -k "radix or tiny_config_all or full_50 or restore" > gpurun_out/r2b/pytest_sort.log 2>&1; echo pytest rc=$?; tail -2 gpurun_out/r2b/pytest_sort.log
timeout 900 python bench.py > gpurun_out/r2b/cfg_lj.json 2> gpurun_out/r2b/cfg_lj.err; echo lj rc=$?
timeout 600 python bench.py --workload tiny --no-multi-source > gpurun_out/r2b/cfg_tiny.json 2> gpurun_out/r2b/cfg_tiny.err; echo tiny rc=$?
OUT=gpurun_out/r2b bash tools/profile_run.sh
timeout 1200 python tools/next2_sweep.py --workload lj --out gpurun_out/r2b/next2_lj.jsonl > gpurun_out/r2b/next2_lj.log 2>&1; echo next2 rc=$?
