# 256-source LJ config: the whole set on one GPU, then every rank's shard of a 2/4/8-GPU run
# (degree-dealt partition, dist.partition_sources), each on one GPU: projected scaling =
# T(256 on 1) / max over ranks T(shard) (plus the 160 KB NCCL broadcast per batch)
run ms256 --sources 256 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
for r in 0 1 2 3 4 5 6 7; do run ms256_s${r}of8 --sources 256 --shard $r/8 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared; done
for r in 0 1 2 3; do run ms256_s${r}of4 --sources 256 --shard $r/4 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared; done
for r in 0 1; do run ms256_s${r}of2 --sources 256 --shard $r/2 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared; done
