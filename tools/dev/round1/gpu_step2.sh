#!/bin/bash
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 900 python -m pytest tests -m gpu -q -x --timeout 600 -k "sortagg" > gpurun_out/pytest_sortagg.log 2>&1; echo pytest-sortagg rc=$?; tail -15 gpurun_out/pytest_sortagg.log
timeout 1200 python -m pytest tests -m gpu -q --timeout 600 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_gpu.log
bash tools/ab_variants.sh
PPR_TRACE=1 timeout 300 python bench.py --steps 2 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/trace.json 2> gpurun_out/trace.err; echo trace rc=$?
timeout 600 python bench.py --mode sortagg --steps 5 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/cfg_sortagg.json 2> gpurun_out/cfg_sortagg.err; echo sortagg rc=$?; tail -c 300 gpurun_out/cfg_sortagg.json; tail -3 gpurun_out/cfg_sortagg.err
