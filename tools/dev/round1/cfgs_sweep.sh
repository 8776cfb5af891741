run orkut_k1e2 --workload orkut --ins 25 --dele 75 --steps 30 --warmup 5 --cpu-budget-s 15
run orkut_k1e3 --workload orkut --ins 250 --dele 750 --steps 20 --warmup 5 --cpu-budget-s 15
run orkut_k1e4 --workload orkut --ins 2500 --dele 7500 --steps 10 --warmup 3 --cpu-budget-s 15
run orkut_k1e5 --workload orkut --ins 25000 --dele 75000 --steps 5 --warmup 3 --no-cpu-baseline
run orkut_k1e6 --workload orkut --ins 250000 --dele 750000 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e
run ms256 --sources 256 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e
