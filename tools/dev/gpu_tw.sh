#!/bin/bash
# Twitter shape: ring-from-seeds (default) vs rounds, with per-round traces
OUT=gpurun_out/tw; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
B="--workload twitter --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-multi-source"
run() { name=$1; shift; timeout 900 python bench.py $B "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g pushes %.4g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['pushes_per_step'], x['iters_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
run tw_default
run tw_rounds --set 7=0
PPR_TRACE=1 run tw_rounds_trace --set 7=0 --steps 2
