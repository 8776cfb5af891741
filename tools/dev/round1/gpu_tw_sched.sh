# Twitter-shaped (no L2 window): ring-from-seeds vs rounds + ring tail, 3 vs 2 edge chains
mkdir -p gpurun_out/twsched
python -m paper_journals_pvldb_guolst17_b200.build >/dev/null || exit 1
b() { name=$1; shift; timeout 900 python bench.py --no-cpu-baseline --no-e2e --workload twitter --steps 5 --warmup 3 "$@" > gpurun_out/twsched/$name.json 2> gpurun_out/twsched/$name.err; python -c "import json;d=json.load(open('gpurun_out/twsched/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f iters %.1f frac %.3f' % (d['ms_per_step'], x['ms_push'], x['iters_per_step'], d['roofline']['frac']))" || tail -3 gpurun_out/twsched/$name.err; }
b auto
PPR_HYBRID_ALL=0 b rounds_tail
PPR_PUSH_U3=0 b ring_u2
PPR_HYBRID_ALL=0 PPR_PUSH_U3=0 b rounds_tail_u2
