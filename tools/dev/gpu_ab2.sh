#!/bin/bash
# A/B of build/variants/libppr_*.so on LJ with u32 and with wide (d_out-carrying) pool entries
mkdir -p gpurun_out/ab2
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
K=${PARITY_K:-"test_tiny_config_all_modes_track_oracle and opt or test_opt_schedules or wide"}
for lib in build/variants/libppr_*.so; do
  name=$(basename $lib .so)
  PPR_LIB=$PWD/$lib timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "$K" > gpurun_out/ab2/pt_$name.log 2>&1
  echo "$name parity: $(tail -1 gpurun_out/ab2/pt_$name.log)"
done
for rep in 1 2; do
for pd in 0 1; do
for lib in build/variants/libppr_*.so; do
  name=$(basename $lib .so)
  PPR_LIB=$PWD/$lib timeout 300 python bench.py --steps 20 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source --pool-degrees $pd ${BENCH_ARGS} > gpurun_out/ab2/b_${name}_$pd_$rep.json 2> gpurun_out/ab2/b_${name}_${pd}_$rep.err
  python -c "import json;d=json.load(open('gpurun_out/ab2/b_${name}_$pd_$rep.json'));x=d['detail'];print('$name pd=$pd', 'step %.3f push %.3f store %.3f edges %.4g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['iters_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 gpurun_out/ab2/b_${name}_${pd}_$rep.err; }
done
done
done
