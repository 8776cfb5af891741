#!/bin/bash
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1200 python -m pytest tests -m gpu -q --timeout 600 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_gpu.log
b() { name=$1; shift; timeout 600 python bench.py --steps 20 --warmup 3 --no-cpu-baseline --no-e2e "$@" > gpurun_out/hy_$name.json 2> gpurun_out/hy_$name.err; python -c "import json;d=json.load(open('gpurun_out/hy_$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.3g pushes %.3g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['pushes_per_step'], x['iters_per_step'], d['roofline']['frac']))" || tail -3 gpurun_out/hy_$name.err; }
for rep in 1 2; do
PPR_HYBRID=0 b lj_h0
b lj_h16k
PPR_HYBRID=4096 b lj_h4k
PPR_HYBRID=65536 b lj_h64k
PPR_HYBRID=0 b lj_e7_h0 --eps 1e-7
b lj_e7_h16k --eps 1e-7
PPR_RELABEL_SPREAD=2 b lj_sp2
PPR_RELABEL_SPREAD=2 b ork_rl1_sp2 --workload orkut --relabel 1
PPR_RELABEL_SPREAD=1 b ork_rl1_sp1 --workload orkut --relabel 1
done
PPR_TRACE=1 timeout 300 python bench.py --steps 2 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/trace_hyb.json 2> gpurun_out/trace_hyb.err; echo trace rc=$?
