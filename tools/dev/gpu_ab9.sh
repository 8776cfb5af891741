#!/bin/bash
# round-end helping: full GPU tests on the help build, LJ/Orkut/ms A/B vs head and the no-help restructure
OUT=gpurun_out/ab9; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
PPR_LIB=$PWD/build/variants/libppr_help.so timeout 1500 python -m pytest tests -m gpu -q -x --timeout 600 > $OUT/pytest_help.log 2>&1; echo "help pytest rc=$? $(tail -1 $OUT/pytest_help.log)"
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 900 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g pushes %.4g frac %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], x['pushes_per_step'], d['roofline']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
for rep in 1 2; do for v in head help nohelp; do run lj_${v}_$rep $v --steps 20 --warmup 5; done; done
for v in head help; do run ork_${v} $v --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3; done
for v in head help; do PPR_TRACE=1 run trace_${v} $v --steps 2 --warmup 3; done
