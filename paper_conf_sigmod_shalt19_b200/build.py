"""Builds libgcgt.so in-tree: sm_100a CUDA (nvcc) + host C++ encoder (g++ -fopenmp).

    python -m paper_conf_sigmod_shalt19_b200.build [--force]
"""
from __future__ import annotations

import os
import subprocess
import sys

HERE = os.path.dirname(os.path.abspath(__file__))
CSRC = os.path.join(HERE, "csrc")
BUILD = os.path.join(HERE, "_build")
LIB = os.path.join(HERE, "libgcgt.so")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]
NCCL_INC = "/usr/include"

SOURCES_CU = ["gcgt.cu"]
SOURCES_CPP = ["encode.cpp"]
HEADERS = ["internal.h", "decode.cuh", "device.cuh", "apps.cuh", "expand.cuh", "bottomup.cuh", "contract.cuh",
           "csr_bfs.cuh"]


def _newer(target, deps):
    if not os.path.exists(target):
        return True
    t = os.path.getmtime(target)
    return any(os.path.getmtime(d) > t for d in deps)


def _run(cmd):
    print("+", " ".join(cmd), flush=True)
    subprocess.check_call(cmd)


def build(force: bool = False, verbose_ptxas: bool = False) -> str:
    os.makedirs(BUILD, exist_ok=True)
    hdrs = [os.path.join(CSRC, h) for h in HEADERS] + [os.path.join(HERE, "..", "include", "gcgt.h")]
    objs = []
    for src in SOURCES_CU:
        s = os.path.join(CSRC, src)
        o = os.path.join(BUILD, src + ".o")
        if force or _newer(o, [s] + hdrs):
            cmd = [NVCC, *ARCH, "-O3", "-lineinfo", "-std=c++17", "-Xcompiler", "-fPIC,-fopenmp", "-c", s, "-o", o]
            if os.environ.get("GCGT_DEV_K"):  # development only: a single zeta_k instantiation
                cmd += [f"-DGCGT_DEV_K={int(os.environ['GCGT_DEV_K'])}"]
            if verbose_ptxas:
                cmd += ["-Xptxas", "-v"]
            _run(cmd)
        objs.append(o)
    for src in SOURCES_CPP:
        s = os.path.join(CSRC, src)
        o = os.path.join(BUILD, src + ".o")
        if force or _newer(o, [s] + hdrs):
            _run(["g++", "-O3", "-std=c++17", "-fopenmp", "-fPIC", "-Wall", "-c", s, "-o", o])
        objs.append(o)
    if force or _newer(LIB, objs):
        _run([NVCC, *ARCH, "-shared", "-o", LIB, *objs, "-Xcompiler", "-fopenmp", "-lgomp"])
    return LIB


if __name__ == "__main__":
    build(force="--force" in sys.argv, verbose_ptxas="-v" in sys.argv)
