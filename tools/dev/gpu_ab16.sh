#!/bin/bash
# new default schedule (ring from the seeds for every graph, lazy done-accounting): full GPU tests + configs
OUT=gpurun_out/ab16; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 1800 python -m pytest tests -m gpu -q -x --timeout 600 > $OUT/pytest.log 2>&1; echo "pytest rc=$? $(tail -1 $OUT/pytest.log)"
run() { name=$1; shift; timeout 900 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f store %.3f edges %.4g frac %.3f l2at %.3f' % (d['ms_per_step'], x['ms_push'], x['ms_store'], x['pushed_edges_per_step'], d['roofline']['frac'], d['roofline_l2_atomics']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
run lj --steps 20 --warmup 5
run lj_rounds --steps 20 --warmup 5 --set 7=0
run tiny --workload tiny --steps 40 --warmup 5
run tiny_rounds --workload tiny --steps 40 --warmup 5 --set 7=0
run ork --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3
run ork100 --workload orkut --ins 25 --dele 75 --steps 20 --warmup 5
run ork100_rounds --workload orkut --ins 25 --dele 75 --steps 20 --warmup 5 --set 7=0
