#!/bin/bash
# lazy-ring knobs retuned with claims a tile ahead
OUT=gpurun_out/ab21; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 600 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f edges %.4g frac %.3f l2at %.3f' % (d['ms_per_step'], x['ms_push'], x['pushed_edges_per_step'], d['roofline']['frac'], d['roofline_l2_atomics']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do for v in base f32 l512 l128; do run lj_${v}_$rep $v --steps 20 --warmup 5; done; done
for v in base f32 l512 l128; do run tiny_${v} $v --workload tiny --steps 40 --warmup 5; done
