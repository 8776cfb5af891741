#!/bin/bash
# dev helper (under gpurun): short benches of several configs
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
run() { name=$1; shift; timeout 900 python bench.py "$@" > gpurun_out/cfg_$name.json 2> gpurun_out/cfg_$name.err; echo "$name rc=$?"; tail -2 gpurun_out/cfg_$name.err;
python - $name <<'PY'
import json,sys
d=json.load(open(f'gpurun_out/cfg_{sys.argv[1]}.json'))
x=d['detail']
print(sys.argv[1], 'value %.4g %s | ms/step %.3f | push %.3f store %.3f restore %.3f | edges/step %.3g iters %.1f | frac %.3f | e2e %s | checks %s | cpu %s' % (d['value'], d['unit'], d['ms_per_step'], x['ms_push'], x['ms_store'], x['ms_restore'], x['pushed_edges_per_step'], x['iters_per_step'], d['roofline']['frac'], d.get('e2e') and round(d['e2e']['ms_per_step'],3), d.get('checks'), d.get('cpu_baseline') and d['cpu_baseline'].get('value')))
PY
}
if [ -n "$CFGFILE" ]; then source "$CFGFILE"; exit 0; fi
run lj --steps 20 --warmup 3 --no-cpu-baseline
