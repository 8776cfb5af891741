# SHARED A/B set: 256 sources on one GPU, rank 0's shard of 8, 16 sources
run ms256 --sources 256 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms256_s0of8 --sources 256 --shard 0/8 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms256_s3of8 --sources 256 --shard 3/8 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms16 --sources 16 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
