#!/bin/bash
# dev helper: GPU tests then short benches of the given modes (run under gpurun)
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 600 python -m pytest tests -m gpu -x -q --timeout 120 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_gpu.log
for m in ${MODES:-opt async}; do
timeout 300 python bench.py --steps 30 --warmup 5 --no-cpu-baseline --mode $m ${BENCH_ARGS} > gpurun_out/bench_$m.json 2> gpurun_out/bench_$m.err; echo bench $m rc=$?; tail -2 gpurun_out/bench_$m.err
python - $m <<'PY'
import json,sys
d=json.load(open(f'gpurun_out/bench_{sys.argv[1]}.json'))
x=d['detail']
print(sys.argv[1], 'value %.3g ms/step %.3f p50 %.3f push %.3f store %.3f iters %.1f edges/step %.3g pushes/step %.3g frac %.3f e2e %s' % (d['value'], d['ms_per_step'], x['ms_per_step_p50'], x['ms_push'], x['ms_store'], x['iters_per_step'], x['pushed_edges_per_step'], x['pushes_per_step'], d['roofline']['frac'], d.get('e2e') and round(d['e2e']['ms_per_step'],3)))
PY
done
