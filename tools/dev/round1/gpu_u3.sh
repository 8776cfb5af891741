mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 900 python -m pytest tests -m gpu -q -x --timeout 600 -k "three_edge or orkut or schedules or undirected" 2>&1 | tail -2
b() { name=$1; shift; timeout 600 python bench.py --no-cpu-baseline --no-e2e "$@" > gpurun_out/u3_$name.json 2> gpurun_out/u3_$name.err; python -c "import json;d=json.load(open('gpurun_out/u3_$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f edges %.3g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['pushed_edges_per_step'], d['roofline']['frac']))" || tail -3 gpurun_out/u3_$name.err; }
for rep in 1 2; do
PPR_PUSH_U3=0 b ork_u2 --workload orkut --steps 10 --warmup 3
b ork_auto --workload orkut --steps 10 --warmup 3
done
PPR_PUSH_U3=0 b tw_u2 --workload twitter --steps 5 --warmup 3
b tw_auto --workload twitter --steps 5 --warmup 3
PPR_PUSH_U3=0 b ork6_u2 --workload orkut --ins 250000 --dele 750000 --steps 4 --warmup 3
b ork6_auto --workload orkut --ins 250000 --dele 750000 --steps 4 --warmup 3
b lj_auto --steps 30 --warmup 3
