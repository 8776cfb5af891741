#!/bin/bash
# ring claim latency: cached tail (TCACHE) and pre-claim
OUT=gpurun_out/ab20; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
for v in tc pretc; do PPR_LIB=$PWD/build/variants/libppr_$v.so timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_configs.py -m gpu -q -x --timeout 300 -k "exactly_once or enqueue_check or schedules or chains or wide or twitter or lj_full or tiny_config_all or multi_source" > $OUT/pt_$v.log 2>&1; echo "$v parity rc=$? $(tail -1 $OUT/pt_$v.log)"; done
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 600 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f edges %.4g frac %.3f l2at %.3f' % (d['ms_per_step'], x['ms_push'], x['pushed_edges_per_step'], d['roofline']['frac'], d['roofline_l2_atomics']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do for v in base tc pretc; do run lj_${v}_$rep $v --steps 20 --warmup 5; done; done
for v in base tc pretc; do run tiny_${v} $v --workload tiny --steps 40 --warmup 5; run ork_${v} $v --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3; done
