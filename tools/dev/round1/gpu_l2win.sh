# Twitter-shaped: persisting-window size A/B (default = min(hot bytes, max window), hit ratio = set-aside / window)
mkdir -p gpurun_out/l2win
python -m paper_journals_pvldb_guolst17_b200.build >/dev/null || exit 1
PPR_DEBUG=1 python -c "
from paper_journals_pvldb_guolst17_b200 import ppr
h = ppr.Ppr(40000000, [0, 1], [1, 0], [0], alpha=0.15, eps=1e-9); h.close()" 2>&1 | grep "L2 window"
b() { name=$1; shift; timeout 900 python bench.py --no-cpu-baseline --no-e2e "$@" > gpurun_out/l2win/$name.json 2> gpurun_out/l2win/$name.err; python -c "import json;d=json.load(open('gpurun_out/l2win/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.3g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], d['roofline']['frac']))" || tail -3 gpurun_out/l2win/$name.err; }
b tw_default --workload twitter --steps 5 --warmup 3
PPR_L2_WIN_MB=${WIN1:-79} b tw_win1 --workload twitter --steps 5 --warmup 3
PPR_L2_WIN_MB=${WIN2:-40} b tw_win2 --workload twitter --steps 5 --warmup 3
PPR_L2_PERSIST=0 b tw_nowin --workload twitter --steps 5 --warmup 3
