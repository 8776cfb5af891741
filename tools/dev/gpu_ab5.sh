#!/bin/bash
# A/B: head vs slab8 (8-byte slab records) on LJ, Orkut k=1e4, multi-source, Twitter; full GPU tests on slab8
OUT=gpurun_out/ab5; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
PPR_LIB=$PWD/build/variants/libppr_slab8.so timeout 1500 python -m pytest tests -m gpu -q -x --timeout 600 > $OUT/pytest_slab8.log 2>&1; echo "slab8 pytest rc=$? $(tail -1 $OUT/pytest_slab8.log)"
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 900 python bench.py --no-cpu-baseline --no-e2e "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g pushes %.4g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['pushes_per_step'], d['roofline']['frac']), ('ms %.2f' % d['multi_source']['ms_per_step']) if 'multi_source' in d else '')" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do for v in head slab8; do run lj_${v}_$rep $v --steps 20 --warmup 5 --no-multi-source; done; done
for v in head slab8; do run ork_${v} $v --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3; done
run ork_slab8_u2 slab8 --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3 --set 8=2
for v in head slab8; do run ms_${v} $v --workload ms-lj --steps 5 --warmup 3; done
for v in head slab8; do run tw_${v} $v --workload twitter --steps 5 --warmup 3; done
