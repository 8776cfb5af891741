#!/bin/bash
# LJ: lazy exchange variants; Twitter: pipe / lean variants (run under gpurun)
OUT=gpurun_out/ab4; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
K="test_tiny_config_all_modes_track_oracle and opt or test_opt_schedules or wide or ring"
for name in base lazy lazy192; do
  PPR_LIB=$PWD/build/variants/libppr_$name.so timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "$K" > $OUT/pt_$name.log 2>&1
  echo "$name parity: $(tail -1 $OUT/pt_$name.log)"
done
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 900 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g pushes %.4g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['pushes_per_step'], x['iters_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do for v in base lazy lazy192; do run lj_${v}_$rep $v --steps 20 --warmup 5; done; done
for v in base nopipe old lazy; do run tw_$v $v --workload twitter --steps 5 --warmup 3; done
