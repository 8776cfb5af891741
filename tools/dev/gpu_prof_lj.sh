#!/bin/bash
# LJ push: per-round trace of two slides + ncu --set full (source counters) of the timed slide 5 push
OUT=gpurun_out/plj; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
B="--steps 3 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source"
PPR_TRACE=1 timeout 300 python bench.py $B > $OUT/trace.json 2> $OUT/trace.err; echo trace rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_push -s 6 -c 1 -o $OUT/push_lj python bench.py $B > $OUT/push_lj.out 2>&1; echo ncu rc=$?
