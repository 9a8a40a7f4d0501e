// Mandelbrot as an index Map: the element is the pixel
// index i (row-major, py outer) and c is computed in the kernel with the same
// window and the same float64-then-round arithmetic as the position vector of
// the plain Map (reading R5), so no position vector is read and the
// counts are bit-identical to the Map over positions.  Loop as mandelbrot.cu
// (eq. (5); reading R4), FMA contraction off.
int mandelbrot_index(int i, int width, int height, int cap) {
    const int px = i % width, py = i / width;
    const float cre = (float)(-2.5 + (double)px * (4.0 / (double)width));
    const float cim = (float)(-1.5 + (double)py * (3.0 / (double)height));
    float x = 0.0f, y = 0.0f;
    int n = 0;
    while (n < cap && x * x + y * y <= 4.0f) {
        float xt = (x * x - y * y) + cre;
        y = (2.0f * x) * y + cim;
        x = xt;
        ++n;
    }
    return n;
}
