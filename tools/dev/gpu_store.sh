#!/bin/bash
# store pipeline check: parity of every store/restore test, LJ bench + launch list, mode ablation edges
OUT=gpurun_out/st; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1200 python -m pytest tests -m gpu -q -x --timeout 600 > $OUT/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 $OUT/pytest_gpu.log
B="--steps 20 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source"
run() { name=$1; shift; timeout 300 python bench.py $B "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f restore %.4f edges %.4g pushes %.4g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['ms_restore'], x['pushed_edges_per_step'], x['pushes_per_step'], x['iters_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
run lj
run lj_t192 
run dup --mode dupdetect
run van --mode vanilla
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $OUT/launches_lj.csv python bench.py --steps 3 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source > $OUT/launches.out 2>&1; echo ncu rc=$?
