#!/bin/bash
# filtered degree refresh of wide pool entries: wide-entry parity tests + Twitter A/B vs head
OUT=gpurun_out/ab10; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
PPR_LIB=$PWD/build/variants/libppr_filt.so timeout 1200 python -m pytest tests -m gpu -q -x --timeout 600 -k "wide or twitter or orkut or growing or forced" > $OUT/pytest_filt.log 2>&1; echo "filt pytest rc=$? $(tail -1 $OUT/pytest_filt.log)"
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 900 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for v in head filt; do run tw_${v} $v --workload twitter --steps 5 --warmup 3; done
for v in head filt; do run lj_${v} $v --steps 10 --warmup 3; done
