#!/bin/bash
mkdir -p gpurun_out/pd
python -m paper_journals_pvldb_guolst17_b200.build || exit 1

REPS=2 PARITY_K="test_tiny_config_all_modes_track_oracle and opt" BENCH_ARGS="--no-multi-source" bash tools/dev/gpu_ab.sh
for lib in build/variants/libppr_*.so; do
  name=$(basename $lib .so)
  PPR_LIB=$PWD/$lib timeout 900 python bench.py --workload twitter --steps 5 --no-cpu-baseline --no-e2e > gpurun_out/pd/tw_$name.json 2> gpurun_out/pd/tw_$name.err
  python -c "import json;d=json.load(open('gpurun_out/pd/tw_$name.json'));x=d['detail'];print('$name twitter', 'step %.2f push %.2f store %.2f edges %.4g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name twitter failed"; tail -3 gpurun_out/pd/tw_$name.err; }
done
