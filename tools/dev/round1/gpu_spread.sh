#!/bin/bash
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
b() { name=$1; shift; timeout 600 python bench.py --steps 20 --warmup 3 --no-cpu-baseline --no-e2e "$@" > gpurun_out/sp_$name.json 2> gpurun_out/sp_$name.err; python -c "import json;d=json.load(open('gpurun_out/sp_$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.3g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['iters_per_step'], d['roofline']['frac']))" || tail -3 gpurun_out/sp_$name.err; }
for rep in 1 2; do
b lj_sp0
PPR_RELABEL_SPREAD=1 b lj_sp1
b ork_rl0 --workload orkut --relabel 0
b ork_rl1 --workload orkut --relabel 1
PPR_RELABEL_SPREAD=1 b ork_rl1_sp1 --workload orkut --relabel 1
done
