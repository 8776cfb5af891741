#!/bin/bash
# Round profile capture (run under gpurun): GPU tests, full default bench,
# ncu launch list of a short bench, ncu --set full of one push launch.
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 900 python -m pytest tests -m gpu -q --timeout 300 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -2 gpurun_out/pytest_gpu.log
timeout 900 python bench.py > gpurun_out/bench_full.json 2> gpurun_out/bench_full.err; echo bench rc=$?
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1; echo ncu-list rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_push -s 4 -c 1 -o gpurun_out/prof_push python bench.py --steps 2 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_full.log 2>&1; echo ncu-full rc=$?
