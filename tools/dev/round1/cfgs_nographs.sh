run lj_nograph --steps 30 --warmup 5 --no-cpu-baseline
run tiny_nograph --workload tiny --steps 40 --warmup 5 --no-cpu-baseline
run orkut100_nograph --workload orkut --ins 25 --dele 75 --steps 30 --warmup 5 --no-cpu-baseline
