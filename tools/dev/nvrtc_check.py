"""Compile one signature kernel from build/obj/jit_src.inc with NVRTC on the CPU box (no GPU needed):
python tools/dev/nvrtc_check.py ["<name expression>"]"""
import ctypes
import re
import sys
import time

inc = open("build/obj/jit_src.inc").read()
names = [x.strip().strip('"') for x in re.search(r"kJitHeaderNames\[\] = \{(.*?)\};", inc, re.S).group(1).split(",")]
bodies = re.findall(r'R"ocl_src\((.*?)\)ocl_src"', inc, re.S)
L = ctypes.CDLL("/usr/local/cuda/lib64/libnvrtc.so.12")
prog = ctypes.c_void_p()
N = len(names)
H = (ctypes.c_char_p * N)(*[b.encode() for b in bodies])
NM = (ctypes.c_char_p * N)(*[n.encode() for n in names])
assert L.nvrtcCreateProgram(ctypes.byref(prog), b'#include "spec_device.cuh"\n', b"ocl_jit.cu", N, H, NM) == 0
expr = (sys.argv[1] if len(sys.argv) > 1 else
        "ocl::k_sga_bulk<ocl::Sig<4, false, 1, 1, 4, false, 6144u, 10244u, 2117u, 2886u, 2056u>, 4, 128, 512, 2>").encode()
L.nvrtcAddNameExpression(prog, expr)
opts = (ctypes.c_char_p * 3)(b"--gpu-architecture=sm_100a", b"-std=c++17", b"-DOCL_JIT=1")
t = time.time()
rc = L.nvrtcCompileProgram(prog, 3, opts)
print("compile rc", rc, "%.2f s" % (time.time() - t))
sz = ctypes.c_size_t()
L.nvrtcGetProgramLogSize(prog, ctypes.byref(sz))
buf = ctypes.create_string_buffer(sz.value)
L.nvrtcGetProgramLog(prog, buf)
print(buf.value.decode()[:4000])
low = ctypes.c_char_p()
if rc == 0:
    L.nvrtcGetLoweredName(prog, expr, ctypes.byref(low))
    cs = ctypes.c_size_t()
    L.nvrtcGetCUBINSize(prog, ctypes.byref(cs))
    print("lowered", low.value, "cubin bytes", cs.value)
