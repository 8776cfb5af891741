#!/bin/bash
# ncu --set full of one push launch on the Twitter- and Orkut-shaped configs (under gpurun)
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:k_push -s 4 -c 1 -o gpurun_out/prof_tw python bench.py --workload twitter --steps 1 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_tw.log 2>&1; echo ncu-tw rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_push -s 4 -c 1 -o gpurun_out/prof_ork python bench.py --workload orkut --steps 1 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_ork.log 2>&1; echo ncu-ork rc=$?
