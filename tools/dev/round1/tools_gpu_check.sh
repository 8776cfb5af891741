#!/bin/bash
# dev helper: build, GPU tests, traced + plain short bench (run under gpurun)
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 600 python -m pytest tests -m gpu -x -q --timeout 120 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_gpu.log
PPR_TRACE=1 timeout 300 python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-e2e ${BENCH_ARGS} > gpurun_out/trace.json 2> gpurun_out/trace.err; echo trace rc=$?
timeout 300 python bench.py --steps 30 --warmup 5 --no-cpu-baseline ${BENCH_ARGS} > gpurun_out/bench_short.json 2> gpurun_out/bench_short.err; echo bench rc=$?
python - <<'PY'
import json
d=json.load(open('gpurun_out/bench_short.json'))
x=d['detail']
print('value %.3g ms/step %.3f p50 %.3f push %.3f store %.3f restore %.3f iters %.1f edges/step %.3g frac %.3f e2e %s' % (d['value'], d['ms_per_step'], x['ms_per_step_p50'], x['ms_push'], x['ms_store'], x['ms_restore'], x['iters_per_step'], x['pushed_edges_per_step'], d['roofline']['frac'], d.get('e2e') and round(d['e2e']['ms_per_step'],3)))
PY
