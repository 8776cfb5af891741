#!/bin/bash
# demand-based slab headroom + runtime slab policy: full GPU tests, LJ/tiny/Orkut k=1e6 A/B vs head
OUT=gpurun_out/ab8; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1500 python -m pytest tests -m gpu -q -x --timeout 600 > $OUT/pytest.log 2>&1; echo "pytest rc=$? $(tail -1 $OUT/pytest.log)"
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 900 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f rebuilds %d edges %.4g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['rebuilds'], x['pushed_edges_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do for v in head cur; do run lj_${v}_$rep $v --steps 20 --warmup 5; done; done
for v in head cur; do run tiny_${v} $v --workload tiny --steps 40 --warmup 5; done
for v in head cur; do run ork6_${v} $v --workload orkut --ins 250000 --dele 750000 --steps 10 --warmup 3; done
