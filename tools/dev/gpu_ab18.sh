#!/bin/bash
# ring default: 3 pipelined chains on LJ, queue-slice size
OUT=gpurun_out/ab18; mkdir -p $OUT
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
run() { name=$1; lib=$2; shift; shift; PPR_LIB=$PWD/build/variants/libppr_$lib.so timeout 600 python bench.py --no-cpu-baseline --no-e2e --no-multi-source "$@" > $OUT/$name.json 2> $OUT/$name.err
  python -c "import json;d=json.load(open('$OUT/$name.json'));x=d['detail'];print('$name', 'step %.3f push %.3f edges %.4g frac %.3f l2at %.3f' % (d['ms_per_step'], x['ms_push'], x['pushed_edges_per_step'], d['roofline']['frac'], d['roofline_l2_atomics']['frac']))" 2>/dev/null || { echo "$name failed"; tail -3 $OUT/$name.err; }; }
PPR_LIB=$PWD/build/variants/libppr_pipeall.so timeout 600 python -m pytest tests/test_gpu_parity.py -m gpu -q -x -k "chains or schedules" > $OUT/pt_pipeall.log 2>&1; echo "pipeall parity $(tail -1 $OUT/pt_pipeall.log)"
for rep in 1 2; do
run lj_base_$rep base --steps 20 --warmup 5
run lj_u3pipe_$rep pipeall --steps 20 --warmup 5 --set 8=3
run lj_qw128_$rep qw128 --steps 20 --warmup 5
run lj_qw512_$rep qw512 --steps 20 --warmup 5
done
run ork_base base --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3
run ork_pipeall pipeall --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3
