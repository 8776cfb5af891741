#!/bin/bash
# under gpurun: full GPU tests + LJ ncu (launch list + --set full of the first timed slide's push)
mkdir -p gpurun_out/tp
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 2400 python -m pytest tests -m gpu -q --timeout 900 > gpurun_out/tp/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -5 gpurun_out/tp/pytest_gpu.log
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/tp/launches_lj.csv python bench.py --steps 3 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source > gpurun_out/tp/launches_lj.json 2>&1; echo ncu-list rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_push -s 6 -c 1 -o gpurun_out/tp/push_lj python bench.py --steps 3 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source > gpurun_out/tp/push_lj.json 2> gpurun_out/tp/push_lj.err; echo ncu-full rc=$?
