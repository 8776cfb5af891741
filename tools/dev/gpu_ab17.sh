#!/bin/bash
# ring claim size (RING_SPLIT, RING_MIN_TILE) on LJ / tiny / Orkut with the ring default
OUT=gpurun_out/ab17; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 600 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f edges %.4g frac %.3f l2at %.3f' % (d['ms_per_step'], x['ms_push'], x['pushed_edges_per_step'], d['roofline']['frac'], d['roofline_l2_atomics']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do for v in base s2 m64 m128 s2m64; do run lj_${v}_$rep $v --steps 20 --warmup 5; done; done
for v in base s2 m64; do run tiny_${v} $v --workload tiny --steps 40 --warmup 5; run ork_${v} $v --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3; done
timeout 900 python bench.py --workload twitter --steps 10 --no-cpu-baseline > $OUT/cfg_twitter.json 2> $OUT/cfg_twitter.err; echo "twitter rc=$?"; python -c "import json;d=json.load(open('$OUT/cfg_twitter.json'));x=d['detail'];print(d['value'], d['ms_per_step'], x['ms_push'], x['ms_store'], d['roofline']['frac'], d['clocks']); print([round(p['ms']-p['ms_push'],1) for p in x['per_step_rank0']])"
timeout 600 python bench.py > $OUT/cfg_lj.json 2> $OUT/cfg_lj.err; echo "lj rc=$?"; python -c "import json;d=json.load(open('$OUT/cfg_lj.json'));print(d['value'], d['ms_per_step'], d['roofline']['frac'], d['clocks'], d['e2e']['value'])"
