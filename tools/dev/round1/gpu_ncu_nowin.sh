#!/bin/bash
# ncu --set full of one push launch: Twitter-shaped and the 8-GPU rank shard, without the L2 window (under gpurun)
mkdir -p gpurun_out/ncu5
python -m paper_journals_pvldb_guolst17_b200.build >/dev/null || exit 1
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:k_push -s 4 -c 1 -o gpurun_out/ncu5/prof_tw python bench.py --workload twitter --steps 1 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu5/ncu_tw.log 2>&1; echo ncu-tw rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_push -s 4 -c 1 -o gpurun_out/ncu5/prof_s0of8 python bench.py --sources 256 --shard 0/8 --mode shared --steps 1 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu5/ncu_s0of8.log 2>&1; echo ncu-shard rc=$?
