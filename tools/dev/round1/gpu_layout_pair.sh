# 16-byte {R, d_out} vertex records (PPR_LAYOUT=packed) vs arrays: parity first, then Twitter/Orkut/LJ
mkdir -p gpurun_out/pair
python -m paper_journals_pvldb_guolst17_b200.build >/dev/null || exit 1
timeout 600 python -m pytest tests -m gpu -q -x --timeout 300 -k "packed or tiny_config_all_modes" > gpurun_out/pair/pytest.log 2>&1; echo pytest rc=$?; tail -2 gpurun_out/pair/pytest.log
b() { name=$1; shift; timeout 900 python bench.py --no-cpu-baseline --no-e2e "$@" > gpurun_out/pair/$name.json 2> gpurun_out/pair/$name.err; python -c "import json;d=json.load(open('gpurun_out/pair/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.3g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], d['roofline']['frac']))" || tail -3 gpurun_out/pair/$name.err; }
PPR_LAYOUT=packed b tw_pair --workload twitter --steps 5 --warmup 3
b tw_soa --workload twitter --steps 5 --warmup 3
PPR_LAYOUT=packed b ork_pair --workload orkut --steps 10 --warmup 3
PPR_LAYOUT=packed b lj_pair --steps 30 --warmup 3
b lj_soa --steps 30 --warmup 3
