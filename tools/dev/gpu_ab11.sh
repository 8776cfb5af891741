#!/bin/bash
# store kernels: launch bounds (fewer waves of warps) -- store parity tests + LJ/tiny store time
OUT=gpurun_out/ab11; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
for v in st_v8a6 st_v6a4; do
  PPR_LIB=$PWD/build/variants/libppr_$v.so timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -x --timeout 600 -k "tiny_config_all_modes or forced or restore or growing or multiset or cancels or radix or multi_source" > $OUT/pt_$v.log 2>&1; echo "$v parity rc=$? $(tail -1 $OUT/pt_$v.log)"
done
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 900 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.4f restore %.4f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['ms_restore'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do for v in st_base st_v8a6 st_v6a4; do run lj_${v}_$rep $v --steps 20 --warmup 5; done; done
for v in st_base st_v8a6 st_v6a4; do run tiny_${v} $v --workload tiny --steps 40 --warmup 5; done
PPR_LIB=$PWD/build/variants/libppr_filt2.so timeout 900 python -m pytest tests -m gpu -q -x --timeout 600 -k "wide or twitter" > $OUT/pt_filt2.log 2>&1; echo "filt2 parity rc=$? $(tail -1 $OUT/pt_filt2.log)"
for v in filt filt2; do run tw_${v} $v --workload twitter --steps 5 --warmup 3; done
