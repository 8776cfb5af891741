#!/bin/bash
# re-entry check: build, full GPU tests, default bench, smoke
mkdir -p gpurun_out/r2d
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1500 python -m pytest tests -m gpu -q --timeout 600 -x > gpurun_out/r2d/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -5 gpurun_out/r2d/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r2d/smoke.log 2>&1; echo smoke rc=$?; tail -2 gpurun_out/r2d/smoke.log
timeout 900 python bench.py > gpurun_out/r2d/bench.json 2> gpurun_out/r2d/bench.err; echo bench rc=$?; tail -c 300 gpurun_out/r2d/bench.err
