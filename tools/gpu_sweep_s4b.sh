# session-4 switch-to-bottom-up sweep at beta = 128 (run under gpurun): vertex-count alpha vs record-bits test
mkdir -p gpurun_out
T="bu_alpha=4 bu_alpha=3 bu_alpha=5 dir_bits=1,alpha_bits=15 dir_bits=1,alpha_bits=30 dir_bits=1,alpha_bits=60"
timeout 600 python tools/sweep.py c2 $T > gpurun_out/sw3_c2.txt 2>&1
timeout 600 python tools/sweep.py c3 $T > gpurun_out/sw3_c3.txt 2>&1
cat gpurun_out/sw3_c2.txt gpurun_out/sw3_c3.txt
