#!/bin/bash
# lazy ring tuning on LJ: async mode and the default schedule
OUT=gpurun_out/ab14; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 600 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f edges %.4g frac %.3f l2at %.3f' % (d['ms_per_step'], x['ms_push'], x['pushed_edges_per_step'], d['roofline']['frac'], d['roofline_l2_atomics']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do for v in f16l128 f16l256 f16l512 f32l256 f8l256; do run async_${v}_$rep $v --steps 20 --warmup 5 --mode async; done; done
for v in f16l256 f32l256; do run def_${v} $v --steps 20 --warmup 5; run ork_${v} $v --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3 --mode async; done
