#!/bin/bash
# under gpurun: build, GPU tests, default bench, then the configs in $CFGFILE
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1200 python -m pytest tests -m gpu -q --timeout 600 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_gpu.log
timeout 900 python bench.py > gpurun_out/bench_full.json 2> gpurun_out/bench_full.err; echo bench rc=$?; tail -c 600 gpurun_out/bench_full.json
[ -n "$CFGFILE" ] && bash tools/bench_configs.sh
