#!/bin/bash
# f3: CGR vs uncompressed CSR on the same machinery (C2, C3)
mkdir -p gpurun_out
T=${TAG:-r2s2ad}
timeout 900 python tools/micro_csr.py c2 4 > gpurun_out/${T}_csr_c2.txt 2>&1
timeout 1200 python tools/micro_csr.py c3 4 > gpurun_out/${T}_csr_c3.txt 2>&1
