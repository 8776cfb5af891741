#!/bin/bash
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -q -x --timeout 300 -k "tiny_config_all_modes_track_oracle and opt or fig or lj_full" > gpurun_out/pytest_wt.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_wt.log
for rep in 1 2; do bash tools/ab_variants.sh; done
PPR_TRACE=1 timeout 300 python bench.py --steps 2 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/trace_wt.json 2> gpurun_out/trace_wt.err; echo trace rc=$?
