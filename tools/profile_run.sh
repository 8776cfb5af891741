#!/bin/bash
# ncu evidence for the bench lines (run under gpurun; one GPU):
#   OUT=<dir> bash tools/profile_run.sh
# For each workload: the launch list of a short bench run, and `ncu --set full` of the push
# launch of the first timed slide (create = launch 0, warm-up slides 1..5, timed slide 0 = launch 6);
# the same run's JSON line gives that slide's pushed edges / pushes (detail.per_step_rank0[0]),
# which tools/dev/traffic.py pairs with the capture's DRAM bytes into profiles/push_traffic.json.
OUT=${OUT:-gpurun_out/prof}
mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
B="--steps 3 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $OUT/launches_lj.csv python bench.py $B > $OUT/launches_lj.out 2>&1; echo lj-list rc=$?
prof() { name=$1; shift; timeout 2400 ncu --set full --clock-control none --import-source on -k regex:k_push -s 6 -c 1 -o $OUT/push_$name python bench.py $B "$@" > $OUT/push_$name.out 2>&1; echo "$name-full rc=$?"; python tools/dev/traffic.py $name $OUT/push_$name.ncu-rep $OUT/push_$name.out 0 --source "profiles/round2_final/push_$name (ncu --set full, push launch of timed slide 5 of bench.py $B $*)" > $OUT/traffic_$name.json 2>&1; }
prof lj
prof orkut --workload orkut --ins 2500 --dele 7500
prof twitter --workload twitter
