#!/bin/bash
# LJ: ring-tail threshold sweep (PPR_OPT_RING_TAIL = 6)
OUT=gpurun_out/tail; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
run() { name=$1; shift; timeout 300 python bench.py --steps 20 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g pushes %.4g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['pushes_per_step'], x['iters_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do
run t16k_$rep
run t4k_$rep --set 6=4096
run t48k_$rep --set 6=49152
run t128k_$rep --set 6=131072
done
