#!/bin/bash
# slab reads with evict_normal on the other shapes + the edge-chain microbenchmark
OUT=gpurun_out/ab7; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 300 ./tools/micro/edge_chain_bench > $OUT/edge_chain_bench.txt 2>&1; echo "micro rc=$?"; cat $OUT/edge_chain_bench.txt
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 900 python bench.py --no-cpu-baseline --no-e2e "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g pushes %.4g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['pushes_per_step'], d['roofline']['frac']), ('ms %.2f' % d['multi_source']['ms_per_step']) if 'multi_source' in d else '')" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for v in base p0s1; do run ork_${v} $v --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3; done
for v in base p0s1; do run ms_${v} $v --workload ms-lj --steps 5 --warmup 3; done
for v in base p0s1; do run tw_${v} $v --workload twitter --steps 5 --warmup 3; done
for v in base p0s1; do run tiny_${v} $v --workload tiny --no-multi-source; done
