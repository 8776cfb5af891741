#!/bin/bash
# Twitter-shaped: NEXT-2 sweep (8 sources per point) and the oracle baseline under a 30-minute cap
mkdir -p gpurun_out/tw
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 2400 python tools/next2_sweep.py --workload twitter --slides 3 --out gpurun_out/tw/next2_twitter.jsonl > gpurun_out/tw/next2_twitter.log 2>&1; echo next2 rc=$?
timeout 2000 python tools/cpu_baselines.py twitter --cap-s 1800 --out gpurun_out/tw/cpu_twitter.jsonl > gpurun_out/tw/cpu_twitter.log 2>&1; echo cpu rc=$?
