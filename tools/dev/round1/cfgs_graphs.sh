run lj_graph --steps 30 --warmup 5 --no-cpu-baseline
run tiny_graph --workload tiny --steps 40 --warmup 5 --no-cpu-baseline
run orkut100_graph --workload orkut --ins 25 --dele 75 --steps 30 --warmup 5 --no-cpu-baseline
