#!/bin/bash
# ncu --set full of one k_push launch (LJ bench) + L2 per-slice balance metrics
mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_push -s 4 -c 1 -o gpurun_out/prof_push python bench.py --steps 2 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_full.log 2>&1; echo ncu-full rc=$?
M=lts__t_sectors_op_atom.sum,lts__t_sectors_op_atom.max,lts__t_sectors_op_atom.avg,lts__t_sectors_op_red.sum,lts__t_sectors_op_red.max,lts__t_sectors_op_red.avg,lts__t_sectors.max,lts__t_sectors.avg,lts__t_sectors.sum,lts__cycles_active.max,lts__cycles_active.avg,l1tex__t_requests_pipe_lsu_mem_global_op_atom.sum,l1tex__t_requests_pipe_lsu_mem_global_op_red.sum,l1tex__t_requests_pipe_lsu_mem_global_op_ld.sum,l1tex__t_sectors_pipe_lsu_mem_global_op_ld.sum,l1tex__data_pipe_lsu_wavefronts.sum,l1tex__lsu_writeback_active.sum,sm__cycles_elapsed.avg,l1tex__throughput.avg.pct_of_peak_sustained_elapsed,lts__throughput.avg.pct_of_peak_sustained_elapsed,lts__t_sectors_srcunit_tex_op_atom.sum,lts__d_sectors_fill_sysmem.sum,lts__average_t_sector_hit_rate_srcunit_tex_op_atom.pct
timeout 600 ncu --metrics $M --clock-control none -k regex:k_push -s 4 -c 1 --csv python bench.py --steps 2 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/ncu_l2.csv 2> gpurun_out/ncu_l2.err; echo ncu-l2 rc=$?
