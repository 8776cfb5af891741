#!/bin/bash
# Every BASELINE config through bench.py on one B200 (run under gpurun):
#   OUT=<dir> bash tools/configs_run.sh
# configs[0] tiny, configs[1] LJ (+ configs[4] 256-source record), configs[2] Orkut
# batch-size sweep k = 1e2..1e6, configs[3] Twitter resident.
OUT=${OUT:-gpurun_out/configs}
mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
run() { name=$1; shift; timeout 1500 python bench.py "$@" > $OUT/cfg_$name.json 2> $OUT/cfg_$name.err; echo "$name rc=$? $(python -c "import json,sys;d=json.load(open('$OUT/cfg_$name.json'));print('%.4g upd/s, %.3f ms/batch, push %.3f ms, store %.3f ms, frac %.3f' % (d['value'], d['ms_per_step'], d['detail']['ms_push'], d['detail']['ms_store'], d['roofline']['frac']))" 2>/dev/null)"; }
run lj
run tiny --workload tiny --no-multi-source
for k in 100 1000 10000 100000 1000000; do
  ni=$(( (k + 3) / 4 )); nd=$(( 3 * k / 4 ))
  st=20; [ $k -ge 1000000 ] && st=10
  run orkut_k$k --workload orkut --ins $ni --dele $nd --steps $st --no-cpu-baseline
done
run twitter --workload twitter --steps 10 --no-cpu-baseline
