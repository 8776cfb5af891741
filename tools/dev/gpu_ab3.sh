#!/bin/bash
# A/B: push variants on LJ + schedule options on the base build
mkdir -p gpurun_out/ab3
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
REPS=2 bash tools/dev/gpu_ab.sh
B="--steps 20 --warmup 5 --no-cpu-baseline --no-e2e --no-multi-source"
run() { name=$1; shift; timeout 300 python bench.py $B "$@" > gpurun_out/ab3/$name.json 2> gpurun_out/ab3/$name.err
  python -c "import json;d=json.load(open('gpurun_out/ab3/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['iters_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 gpurun_out/ab3/$name.err; }; }
run async --mode async
run u3 --set 8=3
run ringall --set 7=1
run notail --set 6=0
