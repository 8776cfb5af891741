#!/bin/bash
mkdir -p gpurun_out/d2
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 300 python tools/dev/diag_restore.py > gpurun_out/d2/diag.txt 2>&1; echo diag rc=$?; cat gpurun_out/d2/diag.txt
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/d2/launches_lj.csv python bench.py --steps 3 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source > gpurun_out/d2/launches_lj.json 2>&1; echo ncu-list rc=$?
