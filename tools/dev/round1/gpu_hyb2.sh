#!/bin/bash
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1200 python -m pytest tests -m gpu -q --timeout 600 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_gpu.log
b() { name=$1; shift; timeout 900 python bench.py --no-cpu-baseline --no-e2e "$@" > gpurun_out/hy_$name.json 2> gpurun_out/hy_$name.err; python -c "import json;d=json.load(open('gpurun_out/hy_$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.3g pushes %.3g iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['pushes_per_step'], x['iters_per_step'], d['roofline']['frac']))" || tail -3 gpurun_out/hy_$name.err; }
b lj --steps 20 --warmup 3
PPR_HYBRID=8192 b lj_8k --steps 20 --warmup 3
PPR_HYBRID=32768 b lj_32k --steps 20 --warmup 3
PPR_HYBRID=0 b lj_h0 --steps 20 --warmup 3
b lj_e7 --eps 1e-7 --steps 20 --warmup 3
b ork --workload orkut --steps 10 --warmup 3
PPR_HYBRID_ALL=0 b ork_all0 --workload orkut --steps 10 --warmup 3
b ork_k1e2 --workload orkut --ins 25 --dele 75 --steps 20 --warmup 3
b ork_k1e6 --workload orkut --ins 250000 --dele 750000 --steps 3 --warmup 3
b tw --workload twitter --steps 5 --warmup 3
PPR_HYBRID_ALL=0 b tw_all0 --workload twitter --steps 5 --warmup 3
