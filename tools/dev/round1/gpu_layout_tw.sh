# Twitter-shaped resident config: SoA arrays vs packed 32-byte vertex records (PPR_LAYOUT=packed)
mkdir -p gpurun_out/layout
python -m paper_journals_pvldb_guolst17_b200.build >/dev/null || exit 1
b() { name=$1; shift; timeout 900 python bench.py --no-cpu-baseline --no-e2e "$@" > gpurun_out/layout/$name.json 2> gpurun_out/layout/$name.err; python -c "import json;d=json.load(open('gpurun_out/layout/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.3g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], d['roofline']['frac']))" || tail -3 gpurun_out/layout/$name.err; }
b tw_soa --workload twitter --steps 5 --warmup 3
PPR_LAYOUT=packed b tw_packed --workload twitter --steps 5 --warmup 3
b ork_soa --workload orkut --steps 10 --warmup 3
PPR_LAYOUT=packed b ork_packed --workload orkut --steps 10 --warmup 3
