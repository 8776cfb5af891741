# relabel spread A/B on the large hot sets (no L2 window): Twitter-shaped and the 8-GPU rank shard
mkdir -p gpurun_out/spread3
python -m paper_journals_pvldb_guolst17_b200.build >/dev/null || exit 1
b() { name=$1; shift; timeout 900 python bench.py --no-cpu-baseline --no-e2e "$@" > gpurun_out/spread3/$name.json 2> gpurun_out/spread3/$name.err; python -c "import json;d=json.load(open('gpurun_out/spread3/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f frac %.3f' % (d['ms_per_step'], x['ms_push'], d['roofline']['frac']))" || tail -3 gpurun_out/spread3/$name.err; }
for sp in 0 1 2; do
PPR_RELABEL_SPREAD=$sp b tw_sp$sp --workload twitter --steps 5 --warmup 3
PPR_RELABEL_SPREAD=$sp b s0of8_sp$sp --sources 256 --shard 0/8 --mode shared --steps 5 --warmup 3
done
b s0of8_norelabel --sources 256 --shard 0/8 --mode shared --steps 5 --warmup 3 --relabel 0
