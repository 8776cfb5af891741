#!/bin/bash
# A/B of build/variants/libppr_*.so: a quick Opt parity check and the LJ bench (run under gpurun)
# env: BENCH_ARGS (extra bench args), REPS (default 2), PARITY_K (pytest -k expr, default tiny opt)
mkdir -p gpurun_out/ab
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
K=${PARITY_K:-"test_tiny_config_all_modes_track_oracle and opt or test_opt_schedules or test_tiny_config_full_50"}
for lib in build/variants/libppr_*.so; do
  name=$(basename $lib .so)
  PPR_LIB=$PWD/$lib timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "$K" > gpurun_out/ab/pt_$name.log 2>&1
  echo "$name parity: $(tail -1 gpurun_out/ab/pt_$name.log)"
done
for rep in $(seq 1 ${REPS:-2}); do
for lib in build/variants/libppr_*.so; do
  name=$(basename $lib .so)
  PPR_LIB=$PWD/$lib timeout 300 python bench.py --steps 20 --warmup 5 --no-cpu-baseline --no-e2e ${BENCH_ARGS} > gpurun_out/ab/b_${name}_$rep.json 2> gpurun_out/ab/b_${name}_$rep.err
  python -c "import json;d=json.load(open('gpurun_out/ab/b_${name}_$rep.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['iters_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 gpurun_out/ab/b_${name}_$rep.err; }
done
done
