#!/bin/bash
# under gpurun: build, full GPU tests, default bench, per-round trace of the LJ push
mkdir -p gpurun_out/chk2
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 2400 python -m pytest tests -m gpu -q --timeout 900 > gpurun_out/chk2/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/chk2/pytest_gpu.log
timeout 900 python bench.py > gpurun_out/chk2/bench.json 2> gpurun_out/chk2/bench.err; echo bench rc=$?; tail -c 300 gpurun_out/chk2/bench.err
PPR_TRACE=1 timeout 300 python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e --no-multi-source > gpurun_out/chk2/trace.json 2> gpurun_out/chk2/trace.err; echo trace rc=$?
