#!/bin/bash
# baseline: LJ bench + per-round trace with the per-CTA time split (run under gpurun)
mkdir -p gpurun_out/base
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 600 python bench.py --steps 30 --warmup 5 --no-cpu-baseline > gpurun_out/base/bench.json 2> gpurun_out/base/bench.err; echo bench rc=$?
PPR_TRACE=1 PPR_LIB=$PWD/build/variants/libppr_split.so timeout 300 python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/base/trace.json 2> gpurun_out/base/trace.err; echo trace rc=$?
nvidia-smi -q | grep -i -A3 "clocks" | head -20 > gpurun_out/base/smi.txt
