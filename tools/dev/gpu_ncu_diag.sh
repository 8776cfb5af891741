#!/bin/bash
# ncu --set full of the LJ push (default build) + A/B of build/variants (run under gpurun)
mkdir -p gpurun_out/diag
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
REPS=1 PARITY_K="test_tiny_config_all_modes_track_oracle and opt" bash tools/dev/gpu_ab.sh
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_push -s 6 -c 1 -o gpurun_out/diag/push_full python bench.py --steps 2 --warmup 5 --no-cpu-baseline --no-e2e > gpurun_out/diag/ncu_full.log 2>&1; echo ncu-full rc=$?
