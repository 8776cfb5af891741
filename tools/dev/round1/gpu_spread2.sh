#!/bin/bash
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1200 python -m pytest tests -m gpu -q --timeout 600 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_gpu.log
b() { name=$1; shift; timeout 600 python bench.py --steps 20 --warmup 3 --no-cpu-baseline --no-e2e "$@" > gpurun_out/sp_$name.json 2> gpurun_out/sp_$name.err; python -c "import json;d=json.load(open('gpurun_out/sp_$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.3g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['iters_per_step'], d['roofline']['frac']))" || tail -3 gpurun_out/sp_$name.err; }
for rep in 1 2; do
PPR_RELABEL_SPREAD=1 b lj_sp1
PPR_RELABEL_SPREAD=2 b lj_sp2
PPR_RELABEL_SPREAD=1 b ork_rl1_sp1 --workload orkut --relabel 1
PPR_RELABEL_SPREAD=2 b ork_rl1_sp2 --workload orkut --relabel 1
done
