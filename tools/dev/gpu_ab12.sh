#!/bin/bash
# tail-tile split (TAILDIV) A/B on LJ + default bench with the NVML clock sampler
OUT=gpurun_out/ab12; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 600 python bench.py > $OUT/bench_default.json 2> $OUT/bench_default.err; echo "default rc=$?"; python -c "import json;d=json.load(open('$OUT/bench_default.json'));print(d['value'], d['ms_per_step'], d['roofline']['frac'], d['clocks'], d['e2e']['value'])"
REPS=2 PARITY_K="test_tiny_config_all_modes_track_oracle and opt or test_opt_schedules or lj_full" BENCH_ARGS="--no-multi-source" bash tools/dev/gpu_ab.sh
