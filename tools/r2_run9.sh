#!/bin/bash
mkdir -p gpurun_out
T=${TAG:-r2j}
timeout 800 python tools/sweep_tunes.py c3 8 "bu_grow=0,bu_alpha=25" "bu_grow=0,bu_alpha=25,nfilter=1" "bu_alpha=50" "bu_alpha=50,nfilter=1" > gpurun_out/${T}_sweep_c3.txt 2>&1
export GCGT_TUNE=graph=0
bash tools/ncu_one.sh ${T}_exp_l7_c3 expand_kernel 7 c3
bash tools/ncu_one.sh ${T}_hub_l7_c3 hub_kernel 7 c3
unset GCGT_TUNE
timeout 600 python tools/sweep_tunes.py c2 8 "bu_grow=0,bu_alpha=25" "bu_grow=0,bu_alpha=25,nfilter=1" > gpurun_out/${T}_sweep_c2.txt 2>&1
